#!/usr/bin/env python
"""Benchmark: fused select -> hash GROUP BY -> aggregate on B200 (BASELINE.json metric).

One step = one pass of the whole hot path (predicate, grouping, aggregation,
finalisation; + allgather/merge when N > 1) over the workload's rows, inputs
already resident in HBM.  Default workload = config C4 (600M-row lineitem,
TPC-H-Q1-style filter + GROUP BY returnflag, linestatus, int64 decimals), the
configuration the north-star target (>= 60% of HBM bandwidth on one B200) is
quoted on.  N > 1 (torchrun): rows are sharded across ranks (fixed total work,
"strong" scaling) and the partial group tables are merged with an NCCL allgather.

    python bench.py [--gpus N] [--steps K] [--warmup W] [--workload c4|c2|c1|c3|c3c|c5] [--impl ours|reference]
"""
from __future__ import annotations

import argparse
import json
import os
import statistics
import sys
import threading
import time

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)

import numpy as np  # noqa: E402
import torch  # noqa: E402

import datagen  # noqa: E402

METRIC = "rows/s and % HBM roofline, fused select+GROUP BY at 1/2/4/8 B200"
Q1_AGGS = [
    {"op": "sum", "a": 0}, {"op": "sum", "a": 1},
    {"op": "sum", "expr": "mul_1minus", "a": 1, "b": 2, "scale": 2},
    {"op": "sum", "expr": "mul_1minus_1plus", "a": 1, "b": 2, "c": 3, "scale": 2},
    {"op": "avg", "a": 0}, {"op": "avg", "a": 1}, {"op": "avg", "a": 2}, {"op": "count"},
]
Q1_PRED = {"hi": datagen.Q1_SHIP_CUTOFF}

WORKLOADS = {
    "c4": dict(desc="C4: lineitem SF100, 600,000,000 rows; TPC-H-Q1-style fused select l_shipdate<=1998-09-02 "
                    "+ GROUP BY (l_returnflag, l_linestatus) = 4 groups; int64 decimal SUM/AVG (int128 exact) + COUNT",
               rows=600_000_000, seed=datagen.BASE_SEED + 4, kind="q1", f64=False, groups=4),
    "c4mm": dict(desc="C4 + MIN/MAX: lineitem SF100, 600,000,000 rows; the Q1-style fused select + GROUP BY "
                      "(l_returnflag, l_linestatus) with MIN(l_quantity) and MAX(l_extendedprice) added to the "
                      "int64 decimal SUM/AVG/COUNT set",
                 rows=600_000_000, seed=datagen.BASE_SEED + 4, kind="q1", f64=False, groups=4, minmax=True),
    "c2": dict(desc="C2: lineitem SF1, 6,000,000 rows; Q1-style 4-group aggregation on fp64 columns with AVG",
               rows=6_000_000, seed=datagen.BASE_SEED + 2, kind="q1", f64=True, groups=4),
    "c1": dict(desc="C1: lineitem SF0.01, 60,000 rows; Q1-style 4 groups, int64 decimals",
               rows=60_000, seed=datagen.BASE_SEED + 1, kind="q1", f64=False, groups=4),
    "c3": dict(desc="C3: lineitem SF10, 60,000,000 rows; GROUP BY l_orderkey (15M groups, HBM hash table), "
                    "COUNT/SUM/MIN/MAX(l_quantity), shuffled row order (seeded Feistel permutation)",
               rows=60_000_000, seed=datagen.BASE_SEED + 3, kind="orderkey", f64=False, groups=15_000_000,
               shuffled=True),
    "c3s": dict(desc="C3 shuffled via sort-based grouping (tier 6): lineitem SF10, 60,000,000 rows in a seeded "
                     "random order; radix sort of (l_orderkey, l_quantity) (P:L456-467) then the sorted-input "
                     "GROUP BY (P:L554-556); COUNT/SUM/MIN/MAX(l_quantity), 15M groups",
                rows=60_000_000, seed=datagen.BASE_SEED + 3, kind="orderkey", f64=False, groups=15_000_000,
                shuffled=True, tier=6),
    "c3c": dict(desc="C3 clustered: lineitem SF10, 60,000,000 rows; GROUP BY l_orderkey (15M groups), "
                     "COUNT/SUM/MIN/MAX(l_quantity), dbgen (clustered, sorted orderkey) row order; sort-based "
                     "grouping of sorted input (P:L554-556)",
                rows=60_000_000, seed=datagen.BASE_SEED + 3, kind="orderkey", f64=False, groups=15_000_000,
                sorted=True),
    "j3": dict(desc="J3 (NEXT-3): PK-FK equi hash join orders.o_orderkey (15,000,000 unique keys, build) x "
                    "lineitem.l_orderkey (60,000,000 rows, probe, dbgen order); direct one-pass PK probe; "
                    "pairs (probe oid, build oid) out",
               rows=60_000_000, seed=datagen.BASE_SEED + 3, kind="join", f64=False, groups=15_000_000),
    "c5": dict(desc="C5 sweep point: 2^28 rows, p i32 ~ U[0,1e6), key = hash(Zipf(s) rank over G), v i64; "
                    "WHERE p < T GROUP BY key: COUNT, SUM, MIN, MAX(v)",
               rows=1 << 28, seed=datagen.BASE_SEED + 5, kind="sweep", f64=False, groups=1 << 10),
}


def q1_fields(f64):
    return (("shipdate", "returnflag", "linestatus") +
            (("quantity_f", "extendedprice_f", "discount_f", "tax_f") if f64 else
             ("quantity", "extendedprice", "discount", "tax")))


def workload_columns(wl, cols):
    """(preds, keys, vals, aggs, bytes_per_row) for a dict of columns."""
    if wl["kind"] == "q1":
        v = ["quantity", "extendedprice", "discount", "tax"]
        if wl["f64"]:
            v = [x + "_f" for x in v]
        aggs = [dict(a, scale=0) if wl["f64"] and a.get("expr", "col") != "col" else a for a in Q1_AGGS]
        if wl.get("minmax"):
            aggs = aggs + [{"op": "min", "a": 0}, {"op": "max", "a": 1}]
        return ([(cols["shipdate"], Q1_PRED)], [cols["returnflag"], cols["linestatus"]], [cols[x] for x in v],
                aggs, 4 + 1 + 1 + 4 * 8)
    aggs = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "min", "a": 0}, {"op": "max", "a": 0}]
    if wl["kind"] == "sweep":
        # the predicate column always, then key and value sectors of 32-byte lines
        # holding a qualifying row: 4 + 16 (1 - (1 - sel)^4) B/row (20 B at 100 %)
        sel = wl["threshold"] / 10**6
        return [(cols["p"], {"hi": wl["threshold"] - 1})], [cols["key"]], [cols["v"]], aggs, \
            4 + 16 * (1 - (1 - sel) ** 4)
    return [], [cols["orderkey"]], [cols["quantity"]], aggs, 16


def wl_fields(wl):
    if wl["kind"] == "sweep":
        return ("p", "key", "v")
    return q1_fields(wl["f64"]) if wl["kind"] == "q1" else ("orderkey", "quantity")


def gen_device(wl, length, start, n, dev):
    if wl["kind"] == "sweep":
        return datagen.sweep_device(length, wl["seed"], wl["groups"], s=wl["zipf"], row0=start, device=dev)
    return datagen.lineitem_device(length, wl["seed"], fields=wl_fields(wl), row0=start, n_total=n,
                                   shuffled=wl.get("shuffled", False), device=dev)


def gen_host(wl, length, start, n, out=None):
    if wl["kind"] == "sweep":
        h = datagen.sweep_host(length, wl["seed"], wl["groups"], s=wl["zipf"], row0=start)
        if out is not None:
            for f in out:
                out[f][:] = h[f]
            return out
        return h
    return datagen.lineitem_host(length, wl["seed"], fields=wl_fields(wl), row0=start, n_total=n,
                                 shuffled=wl.get("shuffled", False), out=out)


class ClockSampler:
    """NVML sampling of SM clock and throttle reasons during the timed region."""

    REASONS = {0x1: "gpu_idle", 0x2: "applications_clocks_setting", 0x4: "sw_power_cap", 0x8: "hw_slowdown",
               0x20: "sw_thermal_slowdown", 0x40: "hw_thermal_slowdown", 0x80: "hw_power_brake_slowdown",
               0x100: "display_clock_setting"}

    def __init__(self, index):
        self.samples, self.reasons, self.ok = [], set(), False
        try:
            import pynvml
            pynvml.nvmlInit()
            self.nv = pynvml
            self.h = pynvml.nvmlDeviceGetHandleByIndex(index)
            self.max_mhz = pynvml.nvmlDeviceGetMaxClockInfo(self.h, pynvml.NVML_CLOCK_SM)
            self.ok = True
        except Exception:  # noqa: BLE001
            self.max_mhz = None
        self._stop = threading.Event()

    def _run(self):
        while not self._stop.is_set():
            try:
                t = time.perf_counter()
                mhz = self.nv.nvmlDeviceGetClockInfo(self.h, self.nv.NVML_CLOCK_SM)
                r = self.nv.nvmlDeviceGetCurrentClocksEventReasons(self.h)
                self.trace.append((t, mhz, r))
            except Exception:  # noqa: BLE001
                pass
            time.sleep(0.0005)

    def start(self):
        """Start sampling (before warm-up, so the thread is running when the timed region opens)."""
        self.trace = []
        if self.ok:
            self.t = threading.Thread(target=self._run, daemon=True)
            self.t.start()
        return self

    def window(self, t0, t1):
        self.t0, self.t1 = t0, t1

    def stop(self):
        self._stop.set()
        if self.ok:
            self.t.join()

    def summary(self):
        """Median SM clock and the union of throttle reasons over samples taken inside the timed window."""
        inside = [(m, r) for t, m, r in self.trace if self.t0 <= t <= self.t1]
        reasons = set()
        for _, r in inside:
            for bit, name in self.REASONS.items():
                if r & bit:
                    reasons.add(name)
        if not inside:
            return {"sm_mhz": None, "sm_max_mhz": self.max_mhz, "reasons": [], "samples": 0}
        return {"sm_mhz": statistics.median(m for m, _ in inside), "sm_max_mhz": self.max_mhz,
                "reasons": sorted(reasons - {"gpu_idle"}), "samples": len(inside)}


def measured_peak_gbs():
    try:
        with open(os.path.join(ROOT, "MEASURED_PEAKS.json")) as f:
            return float(json.load(f)["hbm_gbs"]), "measured (MEASURED_PEAKS.json hbm_gbs)"
    except Exception:  # noqa: BLE001
        return 6650.0, "fallback (B200_PROFILING.md)"


def profiled_traffic(workload, rows):
    """dram read+write bytes per launch of the fused kernel from the committed ncu summary, scaled per row."""
    try:
        with open(os.path.join(ROOT, "profiles", "traffic.json")) as f:
            t = json.load(f)[workload]
        return t["dram_bytes_per_row"] * rows
    except Exception:  # noqa: BLE001
        return None


class pinned_one_core:
    """Run the oracle on ONE host core (sched_setaffinity; SURVEY §8(d) "single-threaded, pinned to 1
    core"); restores the previous affinity."""

    def __enter__(self):
        self.prev = os.sched_getaffinity(0)
        self.core = max(self.prev)
        os.sched_setaffinity(0, {self.core})
        return self.core

    def __exit__(self, *exc):
        os.sched_setaffinity(0, self.prev)


def host_cpu(core):
    model = "unknown"
    try:
        with open("/proc/cpuinfo") as f:
            for line in f:
                if line.startswith("model name"):
                    model = line.split(":", 1)[1].strip()
                    break
    except OSError:
        pass
    return {"pinned_core": core, "host_cores": os.cpu_count(), "cpu_model": model,
            "note": f"1 of {os.cpu_count()} host cores ({model}), pinned with sched_setaffinity"}


def oracle_time(wl, cols, rows):
    import oracle
    p, k, v, a, _ = workload_columns(wl, {f: c[:rows] for f, c in cols.items()})
    t0 = time.perf_counter()
    oracle.sga(p, k, v, a, order_by_key=(wl["kind"] == "q1"))
    return time.perf_counter() - t0


def run_reference(args, wl, rank):
    """--impl reference: the CPU oracle (as it stands, 1 thread) on a bounded sample per step."""
    if rank != 0:
        return
    sample = min(wl["rows"], args.ref_rows)
    cols = gen_host(wl, sample, 0, wl["rows"])
    for _ in range(args.warmup):
        oracle_time(wl, cols, sample)
    with pinned_one_core() as core:
        ts = [oracle_time(wl, cols, sample) for _ in range(args.steps)]
    ms = 1e3 * statistics.mean(ts)
    value = sample / (ms / 1e3)
    desc = f"first {sample:,} rows of the {wl['rows']:,}-row workload per step, oracle.sga single-threaded"
    line = {"impl": "reference", "metric": METRIC, "value": value, "unit": "rows/s", "n_gpus": args.gpus,
            "steps": args.steps, "warmup": args.warmup, "ms_per_step": ms, "higher_is_better": True,
            "scaling": "strong", "vs_baseline": None, "dtype": "int64" if not wl["f64"] else "f64",
            "data": "synthetic (seeded lineitem-shaped generator, datagen/)",
            "config": {"workload": wl["desc"], "rows": wl["rows"], "sample_rows": sample},
            "cpu_baseline": {"value": value, "unit": "rows/s", "cores": 1, "kind": "oracle", "sample": desc,
                             **host_cpu(core)},
            "e2e": {"value": value, "unit": "rows/s", "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0}}
    print(json.dumps(line), flush=True)


def bench_join(args, wl, dev):
    """J3: build + probe per step, device-resident inputs; value = probe rows / step time."""
    import paper_journals_pvldb_heimelspmm13_b200 as ocl
    n = wl["rows"]
    nb = (n + 27) // 28 * 7                          # every order a lineitem block can reference
    probe = datagen.lineitem_device(n, wl["seed"], fields=("orderkey",), device=dev)["orderkey"]
    build_h = datagen.orders_keys(nb)
    build = torch.from_numpy(build_h).to(dev)
    torch.cuda.synchronize()
    state = {}

    def step():
        jb = ocl.JoinBuild(build)
        state["r"] = jb.probe(probe, pk_build=True, out_capacity=n)
        state["jb"] = jb

    clk = ClockSampler(dev.index).start()
    for _ in range(args.warmup):
        step()
    torch.cuda.synchronize()
    op, ob, nout, st = state["r"]
    assert int(st.item()) == 0 and int(state["jb"].status.item()) == 0, "join device status"
    npairs = int(nout.item())
    K = args.steps
    t0, t1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    torch.cuda.synchronize()
    l0 = ocl.launch_count()
    h0 = time.perf_counter()
    t0.record()
    for _ in range(K):
        step()
    t1.record()
    torch.cuda.synchronize()
    h1 = time.perf_counter()
    clk.window(h0, h1)
    clk.stop()
    ms = t0.elapsed_time(t1) / K
    peak, peak_src = measured_peak_gbs()
    algo = 8 * nb + 16 * nb + 8 * n + 8 * npairs      # build keys, table entries, probe keys, pairs out
    cpu = None
    if not args.no_cpu:
        import oracle
        sample = min(n, 20_000_000)
        ph = datagen.lineitem_host(sample, wl["seed"], fields=("orderkey",), n_total=n)["orderkey"]
        tc = time.perf_counter()
        oracle.hash_join(build_h, ph)
        dt = time.perf_counter() - tc
        cpu = {"value": sample / dt, "unit": "rows/s", "cores": 1, "kind": "oracle",
               "sample": f"build all {nb:,} orders keys + probe the first {sample:,} lineitem rows, "
                         f"oracle.hash_join (C++17 unordered_map, single thread), {dt:.1f} s"}
    line = {"metric": METRIC, "value": n / (ms / 1e3), "unit": "rows/s", "n_gpus": 1, "steps": K,
            "warmup": args.warmup, "ms_per_step": ms, "higher_is_better": True, "scaling": "strong",
            "vs_baseline": None, "dtype": "int64", "data": "synthetic (datagen lineitem / orders keys)",
            "config": {"workload": wl["desc"], "rows": n, "build_rows": nb, "pairs": npairs,
                       "l2": "inputs 0.6 GB > 2x L2, no flush needed"},
            "roofline": {"bound": "hbm", "achieved": algo / (ms / 1e3) / 1e9, "peak": peak, "unit": "GB/s",
                         "frac": algo / (ms / 1e3) / 1e9 / peak, "traffic": None,
                         "kernel": "ocl::k_join_insert/alloc/fill + k_join_probe_pk (whole step)",
                         "algorithmic_bytes_per_launch": algo, "peak_source": peak_src},
            "cpu_baseline": cpu, "e2e": None, "gpu_launches": ocl.launch_count() - l0, "clocks": clk.summary()}
    print(json.dumps(line), flush=True)


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=50)
    ap.add_argument("--warmup", type=int, default=3)
    ap.add_argument("--workload", default="c4", choices=sorted(WORKLOADS))
    ap.add_argument("--impl", default="ours", choices=["ours", "reference"])
    ap.add_argument("--ref-rows", type=int, default=20_000_000)
    ap.add_argument("--cpu-rows", type=int, default=200_000_000, help="cpu_baseline sample (rows)")
    ap.add_argument("--e2e-steps", type=int, default=3)
    ap.add_argument("--no-e2e", action="store_true")
    ap.add_argument("--no-cpu", action="store_true")
    ap.add_argument("--tier", type=int, default=0)
    ap.add_argument("--no-sorted", action="store_true", help="c3c: hash grouping instead of the sorted-input path")
    ap.add_argument("--graph", action="store_true", help="replay the fused call as one CUDA graph (1 GPU)")
    ap.add_argument("--c5-groups", type=int, default=1 << 10, help="C5: key cardinality G")
    ap.add_argument("--c5-zipf", type=float, default=0.0, help="C5: Zipf exponent s (0 = uniform)")
    ap.add_argument("--c5-sel", type=float, default=1.0, help="C5: selectivity (0.01, 0.5, 1.0)")
    ap.add_argument("--dist", action="store_true",
                    help="1 GPU: run the distributed path (partial -> NCCL exchange -> merge in the library) on a "
                         "world-size-1 communicator, to measure its overhead (always on for N > 1)")
    ap.add_argument("--jit", action="store_true",
                    help="run the plan through the run-time compiled (NVRTC) signature kernel even when a "
                         "compiled-in signature matches (the path every other plan of the family takes)")
    ap.add_argument("--dist-mode", default="auto", choices=["auto", "allgather", "alltoall"],
                    help="exchange of the distributed path (auto: allgather for partial tables <= 1 MB)")
    args = ap.parse_args()
    wl = dict(WORKLOADS[args.workload])
    if args.no_sorted and wl.get("sorted"):
        wl["sorted"] = False
        wl["desc"] = wl["desc"].replace("sort-based grouping of sorted input (P:L554-556)", "hash grouping")
    if wl["kind"] == "sweep":
        wl.update(groups=args.c5_groups, zipf=args.c5_zipf, threshold=max(1, int(round(args.c5_sel * 10**6))))
        wl["desc"] += f" [G={args.c5_groups}, zipf={args.c5_zipf}, selectivity={args.c5_sel}]"
    if args.jit:
        os.environ["OCL_JIT_ALL"] = "1"
    world = int(os.environ.get("WORLD_SIZE", "1"))
    rank = int(os.environ.get("RANK", "0"))
    local = int(os.environ.get("LOCAL_RANK", "0"))
    if args.impl == "reference":
        run_reference(args, wl, rank)
        return
    torch.cuda.set_device(local)
    dev = torch.device("cuda", local)
    if wl["kind"] == "join":
        if world == 1:
            bench_join(args, wl, dev)
        return
    if world > 1:
        import torch.distributed as dist
        dist.init_process_group("nccl", device_id=dev)
    import paper_journals_pvldb_heimelspmm13_b200 as ocl
    from paper_journals_pvldb_heimelspmm13_b200.distributed import shard_range

    n = wl["rows"]
    start, length = shard_range(n, rank, world)
    cols = gen_device(wl, length, start, n, dev)
    torch.cuda.synchronize()
    p, k, v, aggs, bpr = workload_columns(wl, cols)
    order = wl["kind"] == "q1"
    eg = wl["groups"]
    key_sorted = bool(wl.get("sorted"))
    tier = args.tier or wl.get("tier", 0)
    # multi-GPU: the library exchanges the partial tables itself over an NCCL communicator
    # (ocl_ctx_attach_nccl + ocl_sga_args.distributed; no host sync inside a step)
    distributed = 0
    dctx = None
    if world > 1 or args.dist:
        if world == 1:
            import torch.distributed as dist
            dctx = ocl.Context(local)
            dctx.attach_nccl(ocl.nccl_unique_id(), 0, 1)
        else:
            dctx = ocl.attach_nccl(local)
        probe = ocl.SgaCall(p, k, v, aggs, expected_groups=eg, out_capacity=max(16, 2 * eg), tier=tier,
                            key_sorted=key_sorted)
        small = max(16, 2 * eg) * ocl.partial_row_bytes(probe) <= (1 << 20)
        del probe
        distributed = {"allgather": 1, "alltoall": 2}.get(args.dist_mode, 1 if small else 2)
        order = order and distributed == 1
    call = ocl.SgaCall(p, k, v, aggs, expected_groups=eg, out_capacity=max(16, 2 * eg), order_by_key=order,
                       tier=tier, key_sorted=key_sorted, distributed=distributed, ctx=dctx)
    ctx = call.ctx
    # inputs smaller than 2x the 126 MB L2 are flushed before every step (a 512 MB write)
    flush = torch.empty(512 << 20, dtype=torch.uint8, device=dev) if bpr * length < (256 << 20) else None

    graph = None
    if args.graph and world == 1:
        l0 = ocl.launch_count()
        call.launch()                                    # kernels per call (a replay launches the same ones)
        per_call = ocl.launch_count() - l0
        graph = call.capture()

    def step():
        if graph is not None:
            graph.replay()
        else:
            call.launch()

    clk = ClockSampler(local).start()
    for _ in range(args.warmup):
        step()
    torch.cuda.synchronize()
    keys, outs = call.result()           # raises on a device status error
    G = len(keys)

    K = args.steps
    kev = [(torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)) for _ in range(K)]
    for a, b in kev:               # torch creates the CUDA event lazily: materialise before handing it over
        a.record()
        b.record()
    t0, t1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    sev = [(torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)) for _ in range(K)]
    xev = [(torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)) for _ in range(K)]
    for a, b in xev:
        a.record()
        b.record()
    if world > 1:
        dist.barrier()
    torch.cuda.synchronize()
    launches0 = ocl.launch_count()
    h0 = time.perf_counter()
    t0.record()
    for i in range(K):
        if graph is None:
            ocl.set_kernel_events(ctx, kev[i][0], kev[i][1])
            if distributed:
                ocl.set_phase_events(ctx, 1, xev[i][0], xev[i][1])
        if flush is not None:
            flush.zero_()
        sev[i][0].record()
        step()
        sev[i][1].record()
    t1.record()
    torch.cuda.synchronize()
    h1 = time.perf_counter()
    clk.window(h0, h1)
    clk.stop()
    ocl.set_kernel_events(ctx, None, None)
    ocl.set_phase_events(ctx, 1, None, None)
    kernel_name = ocl.last_kernel(ctx)
    launches = ocl.launch_count() - launches0
    if world > 1:
        dist.barrier()
    # per-step device time: the whole region / K, or (L2 flushed between steps) the mean of per-step events
    ms = t0.elapsed_time(t1) / K if flush is None else statistics.mean(a.elapsed_time(b) for a, b in sev)
    # graph replay: the library's kernel events are not in the graph -> the step events bracket the kernels
    kms = statistics.mean(a.elapsed_time(b) for a, b in (kev if graph is None else sev))
    if graph is not None:
        launches = per_call * K
    xms = statistics.mean(a.elapsed_time(b) for a, b in xev) if distributed and graph is None else None
    if world > 1:
        tt = torch.tensor([ms, kms, xms or 0.0], dtype=torch.float64, device=dev)
        dist.all_reduce(tt, op=dist.ReduceOp.MAX)
        ms, kms, xms = tt.tolist()
    value = n / (ms / 1e3)
    peak, peak_src = measured_peak_gbs()
    out_bytes = G * (8 + sum(o.element_size() * (o[0].numel() if o.dim() > 1 else 1) for o in outs))
    algo_bytes = bpr * length
    achieved = algo_bytes / (kms / 1e3) / 1e9

    # ---- end to end: host (pinned) buffers through the public API, copies inside the timed region
    e2e = None
    if not args.no_e2e:
        host = {f: torch.empty(length, dtype=c.dtype, pin_memory=True) for f, c in cols.items()}
        gen_host(wl, length, start, n, out={f: h.numpy() for f, h in host.items()})
        hp, hk, hv, haggs, _ = workload_columns(wl, host)
        h2d = sum(h.numel() * h.element_size() for h in host.values())
        # ocl_select_group_aggregate_host: pinned host shard -> chunked H2D overlapped with the fused kernel
        # (-> partial exchange + merge over NCCL when distributed) -> D2H of the result; blocking
        hcall = ocl.SgaCall(hp, hk, hv, haggs, expected_groups=eg, out_capacity=max(16, 2 * eg),
                            order_by_key=order, tier=args.tier, host=True, chunk_rows=1 << 24,
                            distributed=distributed, ctx=dctx, device=dev)
        # (the host-buffer entry streams chunks through the one-pass hash kernel, also for sorted input)
        hcall.launch()                                     # warm-up
        ke = max(1, args.e2e_steps)
        if world > 1:
            dist.barrier()
        torch.cuda.synchronize()
        te = time.perf_counter()
        for _ in range(ke):
            hcall.launch()                                 # blocks until results are on the host
        e2e_s = (time.perf_counter() - te) / ke
        if world > 1:
            tt = torch.tensor([e2e_s], dtype=torch.float64, device=dev)
            dist.all_reduce(tt, op=dist.ReduceOp.MAX)
            e2e_s = tt.item()
        hk_, ho_ = hcall.result()
        d2h = 8 + 4 + len(hk_) * 8 + sum(o.numel() * o.element_size() for o in ho_)
        e2e = {"value": n / e2e_s, "unit": "rows/s", "h2d_bytes_per_step": int(h2d),
               "d2h_bytes_per_step": int(d2h), "steps": ke,
               # the host link is the bound end to end: H2D bytes / step time (PCIe Gen5 x16 ~55 GB/s)
               "h2d_gbs": h2d / e2e_s / 1e9,
               "path": "ocl_select_group_aggregate_host (pinned host columns, chunked H2D overlapped with the "
                       "fused kernel" + (", NCCL partial exchange + merge" if distributed else "") +
                       ", D2H of the result)"}

    cpu = None
    if rank == 0 and world == 1 and not args.no_cpu:
        sample = min(n, args.cpu_rows)
        hcols = {f: h.numpy()[:sample] for f, h in host.items()} if e2e is not None else \
            gen_host(wl, sample, 0, n)
        with pinned_one_core() as core:
            dt = oracle_time(wl, hcols, sample)
        cpu = {"value": sample / dt, "unit": "rows/s", "cores": 1, "kind": "oracle",
               "sample": f"first {sample:,} rows of the same workload, oracle.sga (C++17, single thread), "
                         f"{dt:.1f} s", **host_cpu(core)}

    if rank == 0:
        line = {
            "metric": METRIC, "value": value, "unit": "rows/s", "n_gpus": world, "steps": K, "warmup": args.warmup,
            "ms_per_step": ms, "higher_is_better": True, "scaling": "strong", "vs_baseline": None,
            "dtype": "f64" if wl["f64"] else "int64",
            "data": "synthetic (seeded lineitem-shaped generator datagen/, generated in place on each GPU)",
            "config": {"workload": wl["desc"], "rows": n, "rows_per_gpu": length, "groups": G,
                       "bytes_per_row": bpr, "parallelism": f"row-sharded dp{world}",
                       "l2": f"inputs {bpr * length / 1e9:.2f} GB per GPU > 2x the 126 MB L2, no flush needed"
                             if flush is None else "inputs < 2x L2: L2 flushed (512 MB write) before every step, "
                                                   "per-step CUDA events exclude the flush",
                       "launch": "one CUDA graph replay per step" if graph is not None else "stream launches",
                       "grouping": "sort-based (sorted input)" if key_sorted else
                                   ("radix sort + sorted input (tier 6)" if tier == 6 else "hash")},
            "roofline": {"bound": "hbm", "achieved": achieved, "peak": peak, "unit": "GB/s", "frac": achieved / peak,
                         "traffic": profiled_traffic(args.workload, length), "kernel": "ocl::" + kernel_name,
                         "kernel_ms": kms, "algorithmic_bytes_per_launch": algo_bytes, "peak_source": peak_src,
                         # high-G paths also report the bytes including the G output rows
                         "achieved_with_output": (algo_bytes + out_bytes) / (kms / 1e3) / 1e9,
                         "output_bytes_per_launch": out_bytes},
            "hbm_frac_step": algo_bytes / (ms / 1e3) / 1e9 / peak,
            "exchange": None if not distributed else {
                "mode": "allgather" if distributed == 1 else "alltoall", "ms": xms,
                "what": "NCCL exchange of partial tables + merge + finalise inside ocl_select_group_aggregate "
                        "(phase-1 events, max over ranks)", "world": world},
            "cpu_baseline": cpu, "e2e": e2e, "gpu_launches": launches, "clocks": clk.summary(),
        }
        print(json.dumps(line), flush=True)
    if world > 1:
        dist.destroy_process_group()


if __name__ == "__main__":
    main()
