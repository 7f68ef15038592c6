"""Config C5: the group-cardinality sweep on one B200.

n = 2^28 rows of (p i32 ~ U[0,1e6), key = hash(Zipf(s) rank over G), v i64 ~ U[0,1e6)),
WHERE p < T GROUP BY key: COUNT, SUM, MIN, MAX(v) through the library's fused entry
(auto tier).  G in {2^2, 2^4, ..., 2^24}, s in {0, 1.0, 1.5}, T in {1e4, 5e5, 1e6}
(selectivity 1 %, 50 %, 100 %).  Columns are generated on the device once per (G, s);
each point: 2 warm-up calls, then `--steps` calls timed with CUDA events around each
call (the fused kernel or the partitioned passes + finalise, inputs resident).

    python tools/sweep_c5.py [--steps 5] [--out profiles/r01_c5_sweep.json]

Writes one JSON object per point (and a markdown table next to it).  Stream bytes per
row (the §8(d) algorithmic figure) = 4 + 16 * (1 - (1 - sel)^4).
"""
import argparse
import json
import os
import sys

import torch

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import datagen  # noqa: E402
import paper_journals_pvldb_heimelspmm13_b200 as ocl  # noqa: E402

AGGS = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "min", "a": 0}, {"op": "max", "a": 0}]


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--steps", type=int, default=5)
    ap.add_argument("--rows", type=int, default=1 << 28)
    ap.add_argument("--out", default=os.path.join(ROOT, "profiles", "r01_c5_sweep.json"))
    ap.add_argument("--groups", default="2,4,6,8,10,12,14,16,18,20,22,24", help="log2 G values")
    ap.add_argument("--zipf", default="0,1.0,1.5")
    ap.add_argument("--sel", default="0.01,0.5,1.0")
    args = ap.parse_args()
    dev = torch.device("cuda", 0)
    peak = json.load(open(os.path.join(ROOT, "MEASURED_PEAKS.json")))["hbm_gbs"] \
        if os.path.exists(os.path.join(ROOT, "MEASURED_PEAKS.json")) else 8000.0
    n = args.rows
    rows = []
    for lg in [int(x) for x in args.groups.split(",")]:
        G = 1 << lg
        for s in [float(x) for x in args.zipf.split(",")]:
            cols = datagen.sweep_device(n, datagen.BASE_SEED + 5, G, s=s, device=dev)
            torch.cuda.synchronize()
            for sel in [float(x) for x in args.sel.split(",")]:
                T = int(round(sel * 10**6))
                call = ocl.SgaCall([(cols["p"], {"hi": T - 1})], [cols["key"]], [cols["v"]], AGGS,
                                   expected_groups=G, out_capacity=max(16, 2 * G))
                for _ in range(2):
                    call.launch()
                torch.cuda.synchronize()
                keys, outs = call.result()
                ev = [(torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True))
                      for _ in range(args.steps)]
                for a, b in ev:
                    a.record()
                    call.launch()
                    b.record()
                torch.cuda.synchronize()
                ms = sorted(a.elapsed_time(b) for a, b in ev)
                med = ms[len(ms) // 2]
                bpr = 4 + 16 * (1 - (1 - sel) ** 4)
                r = {"log2_groups": lg, "zipf": s, "selectivity": sel, "rows": n, "distinct_groups": int(len(keys)),
                     "ms_median": med, "ms_min": ms[0], "rows_per_s": n / (med * 1e-3),
                     "stream_bytes_per_row": bpr, "hbm_frac": n * bpr / (med * 1e-3) / 1e9 / peak,
                     "kernel": ocl.last_kernel(call.ctx)}
                rows.append(r)
                print(json.dumps(r), flush=True)
                del call
            del cols
            torch.cuda.empty_cache()
    with open(args.out, "w") as f:
        for r in rows:
            f.write(json.dumps(r) + "\n")
    md = os.path.splitext(args.out)[0] + ".md"
    with open(md, "w") as f:
        f.write("# C5 sweep on one B200: 2^28 rows, WHERE p < T GROUP BY key, COUNT/SUM/MIN/MAX(v)\n\n")
        f.write(f"`python tools/sweep_c5.py --steps {args.steps}`; median of the timed calls; G rows/s = "
                "input rows / time; HBM frac = stream bytes (4 + 16(1-(1-sel)^4) B/row) / time / "
                f"{peak:.0f} GB/s.\n\n")
        f.write("| log2 G | zipf | sel | distinct | ms | G rows/s | HBM frac | path |\n|---|---|---|---|---|---|---|---|\n")
        for r in rows:
            k = r["kernel"]
            path = "partitioned" if "part" in k else (k.split(";")[1].strip(" >") if ";" in k else k.split("<")[0])
            f.write(f"| {r['log2_groups']} | {r['zipf']} | {r['selectivity']} | {r['distinct_groups']} | "
                    f"{r['ms_median']:.3f} | {r['rows_per_s'] / 1e9:.1f} | {r['hbm_frac']:.3f} | {path} |\n")


if __name__ == "__main__":
    main()
