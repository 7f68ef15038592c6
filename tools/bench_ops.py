#!/usr/bin/env python
"""Per-operator measurements of the unfused chain on one B200.

For every C-ABI operator: device time (CUDA events, median of K launches after warm-up,
inputs resident, inputs >> L2) and the fraction of the measured HBM copy bandwidth its
algorithmic bytes reach.  Workload: config C4 columns (600M lineitem rows, Q1) unless
--rows says otherwise.  Writes one JSON object (stdout and --out)."""
from __future__ import annotations

import argparse
import json
import os
import statistics
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import torch  # noqa: E402

import datagen  # noqa: E402
import paper_journals_pvldb_heimelspmm13_b200 as ocl  # noqa: E402


def timed(fn, steps, warmup):
    for _ in range(warmup):
        fn()
    torch.cuda.synchronize()
    ts = []
    for _ in range(steps):
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record()
        fn()
        b.record()
        torch.cuda.synchronize()
        ts.append(a.elapsed_time(b))
    return statistics.median(ts)


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--rows", type=int, default=600_000_000)
    ap.add_argument("--steps", type=int, default=10)
    ap.add_argument("--warmup", type=int, default=3)
    ap.add_argument("--out", default=None)
    ap.add_argument("--only", default=None, help="run only operators whose name contains this string")
    args = ap.parse_args()
    peak = json.load(open(os.path.join(ROOT, "MEASURED_PEAKS.json")))["hbm_gbs"] if os.path.exists(
        os.path.join(ROOT, "MEASURED_PEAKS.json")) else 6650.0
    n = args.rows
    dev = torch.device("cuda", 0)
    c = datagen.lineitem_device(n, datagen.BASE_SEED + 4, device=dev)
    torch.cuda.synchronize()
    res = {"rows": n, "peak_gbs": peak, "ops": {}}

    def want(name):
        return args.only is None or args.only in name

    def record(name, ms, algo_bytes, note):
        gbs = algo_bytes / (ms / 1e3) / 1e9
        res["ops"][name] = {"ms": ms, "algorithmic_bytes": algo_bytes, "gbs": gbs, "frac": gbs / peak,
                            "rows_per_s": n / (ms / 1e3), "note": note}

    pred = {"hi": datagen.Q1_SHIP_CUTOFF}
    words = (n + 31) // 32
    bm = torch.empty(words, dtype=torch.int32, device=dev)
    # a1: select -> bitmap over i32 / u8 / i64 columns
    if want("a1"):
        ms = timed(lambda: ocl.select_bitmap(c["shipdate"], pred, out=bm), args.steps, args.warmup)
        record("a1_select_bitmap_i32", ms, n * 4 + words * 4, "l_shipdate <= 10471")
        ms = timed(lambda: ocl.select_bitmap(c["returnflag"], {"lo": ord("N"), "hi": ord("N")}, out=bm), args.steps,
                   args.warmup)
        record("a1_select_bitmap_u8", ms, n * 1 + words * 4, "l_returnflag = 'N'")
        ms = timed(lambda: ocl.select_bitmap(c["extendedprice"], {"lo": 1_000_000, "hi": 5_000_000}, out=bm),
                   args.steps, args.warmup)
        record("a1_select_bitmap_i64", ms, n * 8 + words * 4, "1e6 <= l_extendedprice <= 5e6")
    if want("A2"):
        bm2 = ocl.select_bitmap(c["tax"], {"lo": 4})
        out = torch.empty_like(bm)
        ms = timed(lambda: ocl.bitmap_combine("and", bm, bm2, n, out=out), args.steps, args.warmup)
        record("A2_bitmap_combine_and", ms, 3 * words * 4, "two bitmaps -> one")
    # a2: prefix compaction of the Q1 bitmap (selectivity 0.986)
    q1 = ocl.select_bitmap(c["shipdate"], pred)
    oids, m = ocl.prefix_compact(q1, n)
    torch.cuda.synchronize()
    mm = int(m.item())
    if want("a2"):
        ms = timed(lambda: ocl.prefix_compact(q1, n), args.steps, args.warmup)
        record("a2_prefix_compact", ms, words * 4 + mm * 4, f"m = {mm}")
    if want("a3"):
        ms = timed(lambda: ocl.gather(c["extendedprice"], oids, m, max_m=mm), args.steps, args.warmup)
        record("a3_gather_i64", ms, mm * (4 + 8 + 8), "ascending oids, 98.6% dense")
    if want("a4"):
        ms = timed(lambda: ocl.group_build([c["returnflag"], c["linestatus"]], oids=oids, m=m, max_rows=mm,
                                           expected_groups=4, out_capacity=16), args.steps, args.warmup)
        record("a4_group_build_2xu8", ms, mm * (4 + 1 + 1 + 4), "gid column written, 4 groups")
    gids, keys, ng, st = ocl.group_build([c["returnflag"], c["linestatus"]], oids=oids, m=m, max_rows=mm,
                                         expected_groups=4, out_capacity=16)
    # a7-a8: grouped aggregation of the Q1 set over the gids
    vals = [c["quantity"], c["extendedprice"], c["discount"], c["tax"]]
    aggs = [{"op": "sum", "a": 0}, {"op": "sum", "a": 1},
            {"op": "sum", "expr": "mul_1minus", "a": 1, "b": 2, "scale": 2},
            {"op": "sum", "expr": "mul_1minus_1plus", "a": 1, "b": 2, "c": 3, "scale": 2},
            {"op": "avg", "a": 0}, {"op": "avg", "a": 1}, {"op": "avg", "a": 2}, {"op": "count"}]
    if want("a7"):
        ms = timed(lambda: ocl.group_aggregate(gids, ng, 16, vals, aggs, oids=oids, m=m, max_rows=mm), args.steps,
                   args.warmup)
        record("a7_group_aggregate_q1", ms, mm * (4 + 4 + 32), "Q1 aggregates via gids, values gathered at oids")
    chain = sum(res["ops"][k]["ms"] for k in ("a1_select_bitmap_i32", "a2_prefix_compact", "a4_group_build_2xu8",
                                              "a7_group_aggregate_q1") if k in res["ops"])
    # a9: the fused path on the same columns
    call = ocl.SgaCall([(c["shipdate"], pred)], [c["returnflag"], c["linestatus"]], vals, aggs, expected_groups=4,
                       out_capacity=16, order_by_key=True)
    if want("a9"):
        ms = timed(call.launch, args.steps, args.warmup)
        record("a9_fused_select_group_aggregate", ms, n * 38, "one pass, 38 B/row")
        res["unfused_chain_ms"] = chain
        res["fused_speedup_over_chain"] = chain / ms
    line = json.dumps(res, indent=1)
    print(line)
    if args.out:
        with open(args.out, "w") as f:
            f.write(line + "\n")


if __name__ == "__main__":
    main()
