"""Parity at BASELINE.json's full sizes, in the launch configuration bench.py times.

C4 (600M rows, Q1, int64 decimals) and C3 (60M rows, GROUP BY orderkey, ~15M groups) are
generated on the device by datagen (as bench.py does) and compared against the CPU oracle run
over the identical host-generated rows — every output value, not a sample (the oracle finishes
C4 in ~30 s single-threaded)."""
import numpy as np
import pytest
import torch

import datagen
import oracle
from tests._common import Q1_AGGS, Q1_PRED, assert_results_equal_np

pytestmark = [pytest.mark.gpu, pytest.mark.slow]
ocl = pytest.importorskip("paper_journals_pvldb_heimelspmm13_b200")


def _run(wl_rows, seed, fields, build, expected_groups, order_by_key, tier=0):
    dev = torch.device("cuda", 0)
    d = datagen.lineitem_device(wl_rows, seed, fields=fields, device=dev)
    p, k, v, a = build(d)
    call = ocl.SgaCall(p, k, v, a, expected_groups=expected_groups, out_capacity=max(16, 2 * expected_groups),
                       order_by_key=order_by_key, tier=tier)
    call.launch()
    keys, outs = call.result()
    gk, go = keys.cpu().numpy(), [o.cpu().numpy() for o in outs]
    del d, call
    torch.cuda.empty_cache()
    h = datagen.lineitem_host(wl_rows, seed, fields=fields)
    p, k, v, a = build(h)
    rk, ro = oracle.sga(p, k, v, a, order_by_key=order_by_key)
    return gk, go, rk, ro, a, [c.dtype if hasattr(c, "dtype") else None for c in v]


def _q1(c):
    vals = [c["quantity"], c["extendedprice"], c["discount"], c["tax"]]
    return [(c["shipdate"], Q1_PRED)], [c["returnflag"], c["linestatus"]], vals, Q1_AGGS


def test_c4_full_600m_rows():
    fields = ("shipdate", "returnflag", "linestatus", "quantity", "extendedprice", "discount", "tax")
    gk, go, rk, ro, a, _ = _run(600_000_000, datagen.BASE_SEED + 4, fields, _q1, 4, True)
    assert gk.tolist() == rk.tolist() and len(rk) == 4
    assert_results_equal_np(gk, go, rk, ro, a, [np.dtype(np.int64)] * 4)


def test_c3_full_60m_rows_15m_groups():
    fields = ("orderkey", "quantity")
    aggs = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "min", "a": 0}, {"op": "max", "a": 0}]

    def build(c):
        return [], [c["orderkey"]], [c["quantity"]], aggs
    gk, go, rk, ro, a, _ = _run(60_000_000, datagen.BASE_SEED + 3, fields, build, 15_000_000, False)
    assert len(rk) == 15_000_000
    assert_results_equal_np(gk, go, rk, ro, a, [np.dtype(np.int64)])
