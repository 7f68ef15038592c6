"""Repeat the Q1-signature plan under every OCL_BULK config and report mismatches vs the oracle (debug aid)."""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__)))))
import numpy as np
import torch

import datagen
import oracle
import paper_journals_pvldb_heimelspmm13_b200 as ocl
from tests._common import Q1_AGGS, Q1_AGGS_F64, by_key

n = int(sys.argv[1]) if len(sys.argv) > 1 else 3 * 148 * 2048 + 1017
reps = int(sys.argv[2]) if len(sys.argv) > 2 else 5
cfgs = sys.argv[3].split(",") if len(sys.argv) > 3 else ["1", "2", "3", "4", "5", "6", "7"]
for f64 in (False, True):
    li = datagen.lineitem_host(n, datagen.BASE_SEED + 2, fields=datagen.LINEITEM_INT_FIELDS + datagen.LINEITEM_F64_FIELDS)
    vn = ["quantity", "extendedprice", "discount", "tax"]
    vals = [li[x + ("_f" if f64 else "")] for x in vn]
    aggs = Q1_AGGS_F64 if f64 else Q1_AGGS
    preds = [(li["shipdate"], {"hi": 10471})]
    keys = [li["returnflag"], li["linestatus"]]
    rk, routs = oracle.sga(preds, keys, vals, aggs, order_by_key=True)
    d = lambda a: torch.from_numpy(np.ascontiguousarray(a)).cuda()
    dp, dk, dv = [(d(c), s) for c, s in preds], [d(c) for c in keys], [d(c) for c in vals]
    for cfg in cfgs:
        os.environ["OCL_BULK"] = cfg
        bad = 0
        for r in range(reps):
            k, outs, _ = ocl.select_group_aggregate(dp, dk, dv, aggs, expected_groups=4, order_by_key=True)
            cnt = outs[-1].cpu().numpy()
            if not np.array_equal(cnt, routs[-1]):
                bad += 1
                print(f"  f64={f64} cfg={cfg} rep={r}: count {cnt.tolist()} vs {routs[-1].tolist()}  kernel={ocl.last_kernel(ocl.context())}")
        print(f"f64={f64} cfg={cfg}: {bad}/{reps} bad  ({ocl.last_kernel(ocl.context())})", flush=True)
