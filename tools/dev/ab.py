"""A/B timing of library builds (OCL_LIB_PATH) on the bench workloads: fused call time with CUDA events,
median of K calls after warm-up.  Usage: python tools/dev/ab.py <workload spec>... ; each spec is
c4 | c2 | c4mm | c5:G[:zipf[:sel]]."""
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__)))))
import torch

import datagen
import paper_journals_pvldb_heimelspmm13_b200 as ocl
from bench import Q1_AGGS, Q1_PRED

dev = torch.device("cuda", 0)
K = int(os.environ.get("AB_STEPS", "20"))
cache = {}


def q1(n, seed, f64, mm=False):
    key = ("q1", n, f64)
    if key not in cache:
        f = ("shipdate", "returnflag", "linestatus") + (("quantity_f", "extendedprice_f", "discount_f", "tax_f")
                                                        if f64 else ("quantity", "extendedprice", "discount", "tax"))
        cache[key] = datagen.lineitem_device(n, seed, fields=f, device=dev)
    c = cache[key]
    v = ["quantity", "extendedprice", "discount", "tax"]
    v = [x + "_f" for x in v] if f64 else v
    aggs = [dict(a, scale=0) if f64 and a.get("expr", "col") != "col" else a for a in Q1_AGGS]
    if mm:
        aggs = aggs + [{"op": "min", "a": 0}, {"op": "max", "a": 1}]
    return [(c["shipdate"], Q1_PRED)], [c["returnflag"], c["linestatus"]], [c[x] for x in v], aggs, 4


def c5(G, zipf, sel):
    key = ("c5", G, zipf)
    if key not in cache:
        cache.clear()
        torch.cuda.empty_cache()
        cache[key] = datagen.sweep_device(1 << 28, datagen.BASE_SEED + 5, G, s=zipf, device=dev)
    c = cache[key]
    aggs = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "min", "a": 0}, {"op": "max", "a": 0}]
    return [(c["p"], {"hi": int(round(sel * 10**6)) - 1})], [c["key"]], [c["v"]], aggs, G


def run(spec):
    parts = spec.split(":")
    if parts[0] == "c4":
        p, k, v, a, G = q1(600_000_000, datagen.BASE_SEED + 4, False)
    elif parts[0] == "c4mm":
        p, k, v, a, G = q1(600_000_000, datagen.BASE_SEED + 4, False, mm=True)
    elif parts[0] == "c2":
        p, k, v, a, G = q1(6_000_000, datagen.BASE_SEED + 2, True)
    else:
        G = int(parts[1])
        p, k, v, a, G = c5(G, float(parts[2]) if len(parts) > 2 else 0.0, float(parts[3]) if len(parts) > 3 else 1.0)
    call = ocl.SgaCall(p, k, v, a, expected_groups=G, out_capacity=max(16, 2 * G))
    for _ in range(3):
        call.launch()
    call.result()
    ev = [(torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)) for _ in range(K)]
    for s, e in ev:
        s.record()
        call.launch()
        e.record()
    torch.cuda.synchronize()
    ms = statistics.median(s.elapsed_time(e) for s, e in ev)
    print(f"{os.path.basename(ocl.LIB_PATH):28s} {spec:16s} {ms:8.4f} ms  {ocl.last_kernel(call.ctx)}", flush=True)


for spec in sys.argv[1:]:
    run(spec)
