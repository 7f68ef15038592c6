"""Sorted-input GROUP BY (§4.1.6) through the C ABI
vs the CPU oracle.

Group ids on sorted input are fixed by the method (the g-th distinct key has id g), so
gids, keys_out and output row order are compared bit-exactly; aggregates follow the
usual rules (integers / MIN / MAX exact, fp64 SUM / AVG within 1e-9 relative).
"""
import numpy as np
import pytest
import torch

import datagen
import oracle
from tests._common import Q1_AGGS, assert_results_equal, by_key

pytestmark = pytest.mark.gpu

ocl = pytest.importorskip("paper_journals_pvldb_heimelspmm13_b200")
DEV = torch.device("cuda", 0)
UNIT = 2048                       # rows per warp unit of the fused sorted kernels


def dev(a):
    return torch.from_numpy(np.ascontiguousarray(a)).to(DEV)


def sorted_keys(rng, n, mean_run, dtype=np.int64, lo=0):
    """Non-decreasing keys with geometric run lengths (mean mean_run)."""
    if n == 0:
        return np.zeros(0, dtype)
    starts = rng.random(n) < 1.0 / mean_run
    starts[0] = True
    return (np.cumsum(starts) - 1 + lo).astype(dtype)


# ---------------------------------------------------------------- unfused: ocl_group_build_sorted
@pytest.mark.parametrize("n", [0, 1, 31, 32, 33, 2047, 2048, 2049, 65536 + 17, (1 << 20) + 17])
@pytest.mark.parametrize("mean_run", [1.0, 4.0, 1000.0])
def test_group_build_sorted(n, mean_run):
    rng = np.random.default_rng(n + int(mean_run))
    keys = sorted_keys(rng, n, mean_run, lo=-3 if mean_run > 1 else 0)
    keys = np.where(keys < 0, 0, keys).astype(np.int64)   # unsigned packed order: keep non-negative
    ref_g, ref_k = oracle.group_sorted([keys])
    gids, kout, ng, st = ocl.group_build_sorted([dev(keys)])
    torch.cuda.synchronize()
    assert int(st.item()) == 0
    assert int(ng.item()) == len(ref_k)
    assert np.array_equal(gids[:n].cpu().numpy(), ref_g)             # labels fixed by the method
    assert np.array_equal(kout[:len(ref_k)].cpu().numpy(), ref_k)


def test_group_build_sorted_oids_m_and_two_keys():
    rng = np.random.default_rng(5)
    n = 300000
    a = np.sort(rng.integers(0, 7, n)).astype(np.uint8)
    b = np.concatenate([np.sort(rng.integers(0, 200, int((a == v).sum()))) for v in range(7)]).astype(np.uint8)
    oids = np.flatnonzero(rng.random(n) < 0.4).astype(np.uint32)
    ref_g, ref_k = oracle.group_sorted([a, b], oids)
    m = dev(np.array([len(oids)], np.int64))
    pad = np.concatenate([oids, np.zeros(1000, np.uint32)])              # max_rows > m: rows >= m ignored
    gids, kout, ng, st = ocl.group_build_sorted([dev(a), dev(b)], oids=dev(pad.view(np.int32)), m=m,
                                                max_rows=len(pad), out_capacity=len(oids))
    torch.cuda.synchronize()
    assert int(st.item()) == 0 and int(ng.item()) == len(ref_k)
    assert np.array_equal(gids[:len(oids)].cpu().numpy(), ref_g)
    assert np.array_equal(kout[:len(ref_k)].cpu().numpy(), ref_k)


def test_group_build_sorted_status():
    keys = np.arange(10000, dtype=np.int64)
    keys[7777] = 3                                                      # one decreasing step
    _, _, _, st = ocl.group_build_sorted([dev(keys)])
    torch.cuda.synchronize()
    assert int(st.item()) == ocl.OCL_ERR_INVALID_ARG
    keys = np.arange(10000, dtype=np.int64)
    _, _, ng, st = ocl.group_build_sorted([dev(keys)], out_capacity=100)
    torch.cuda.synchronize()
    assert int(st.item()) == ocl.OCL_ERR_CAPACITY and int(ng.item()) == 10000


# ---------------------------------------------------------------- fused: key_sorted
C3_AGGS = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "min", "a": 0}, {"op": "max", "a": 0}]


def _check_sorted(preds, keys, vals, aggs, rtol=1e-9, bitmap=False, out_capacity=None):
    k, outs, bm = ocl.select_group_aggregate([(dev(c), s) for c, s in preds], [dev(c) for c in keys],
                                             [dev(c) for c in vals], aggs, key_sorted=True, bitmap=bitmap,
                                             out_capacity=out_capacity)
    rk, routs = oracle.sga(preds, keys, vals, aggs, order_by_key=True)
    assert np.array_equal(k.cpu().numpy(), rk)                         # key order = gid order
    dts = [c.dtype for c in vals]
    assert_results_equal(by_key(k.cpu().numpy(), [o.cpu().numpy() for o in outs], aggs, dts),
                         by_key(rk, routs, aggs, dts), aggs, dts, rtol=rtol)
    if bitmap:
        n = len(preds[0][0])
        ref = np.full((n + 31) // 32, 0xFFFFFFFF, np.uint32)
        for c, s in preds:
            ref &= oracle.select(c, s)
        if n % 32:
            ref[-1] &= (1 << (n % 32)) - 1
        assert np.array_equal(bm.cpu().numpy().view(np.uint32)[:len(ref)], ref)
    return k, outs


@pytest.mark.parametrize("n", [1, 63, 64, 65, UNIT - 1, UNIT, UNIT + 1, 3 * UNIT + 5, 400000, (1 << 20) + 17])
def test_fused_sorted_c3_shape(n):
    """C3 clustered (dbgen order): GROUP BY l_orderkey, COUNT/SUM/MIN/MAX(l_quantity); with and without
    the Q1 shipdate predicate (static shapes key i64 / pred i32 + key i64)."""
    li = datagen.lineitem_host(n, datagen.BASE_SEED + 3)
    _check_sorted([], [li["orderkey"]], [li["quantity"]], C3_AGGS)
    _check_sorted([(li["shipdate"], {"hi": 9500})], [li["orderkey"]], [li["quantity"]], C3_AGGS, bitmap=True)


@pytest.mark.parametrize("mean_run,sel", [(1.0, 1.0), (3.0, 0.5), (50.0, 0.9), (5000.0, 1.0), (1e9, 1.0),
                                          (1e9, 0.01), (200.0, 0.005), (UNIT, 0.3)])
def test_fused_sorted_runs_and_selectivity(mean_run, sel):
    """Runs shorter than a lane pair up to one run over all rows (chains across many units); low
    selectivity leaves whole units empty between the pieces of a run."""
    rng = np.random.default_rng(int(mean_run) % 1000 + int(sel * 100))
    n = 300000
    keys = sorted_keys(rng, n, mean_run)
    p = rng.integers(0, 10**6, n).astype(np.int32)
    v = rng.integers(-10**6, 10**6, n).astype(np.int64)
    _check_sorted([(p, {"hi": int(sel * 10**6) - 1})], [keys], [v], C3_AGGS)


def test_fused_sorted_generic_plans():
    """DynShape instantiations: two u8 keys with the Q1 aggregate set (int expressions, AVG), fp64
    values, mixed int/fp64 values, values beyond int32 (exact int128 path), the key ~0."""
    rng = np.random.default_rng(9)
    n = 250000
    a = np.sort(rng.integers(60, 90, n)).astype(np.uint8)
    b = np.concatenate([np.sort(rng.integers(0, 256, int((a == x).sum()))) for x in range(60, 90)]).astype(np.uint8)
    sd = rng.integers(8000, 11000, n).astype(np.int32)
    qty = rng.integers(1, 51, n).astype(np.int64) * 100
    price = rng.integers(90000, 10**7, n).astype(np.int64)
    disc = rng.integers(0, 11, n).astype(np.int64)
    tax = rng.integers(0, 9, n).astype(np.int64)
    pred = [(sd, {"hi": 10471})]
    _check_sorted(pred, [a, b], [qty, price, disc, tax], Q1_AGGS)
    f = [x.astype(np.float64) / 100.0 for x in (qty, price, disc, tax)]
    aggs_f = [dict(x, scale=0) for x in Q1_AGGS] + [{"op": "min", "a": 1}, {"op": "max", "a": 1}]
    _check_sorted(pred, [a, b], f, aggs_f)
    big = rng.integers(-2**62, 2**62, n).astype(np.int64)              # SUM beyond int64, MIN/MAX beyond int32
    mixed = [big, f[1]]
    aggs_m = [{"op": "sum", "a": 0}, {"op": "min", "a": 0}, {"op": "max", "a": 0}, {"op": "avg", "a": 0},
              {"op": "sum", "a": 1}, {"op": "avg", "a": 1}, {"op": "count"}]
    _check_sorted(pred, [a, b], mixed, aggs_m)
    keys = sorted_keys(rng, n, 40.0)
    keys[-5000:] = -1                                                   # ~0: largest unsigned packed key
    _check_sorted([], [keys], [qty], C3_AGGS)


def test_fused_sorted_edge_cases():
    rng = np.random.default_rng(3)
    n = 100000
    keys = sorted_keys(rng, n, 7.0)
    v = rng.integers(0, 100, n).astype(np.int64)
    p = rng.integers(0, 100, n).astype(np.int32)
    k, outs, _ = ocl.select_group_aggregate([(dev(p), {"lo": 200})], [dev(keys)], [dev(v)], C3_AGGS,
                                            key_sorted=True)
    assert k.numel() == 0                                               # empty selection: G = 0 (s17)
    base = dev(np.concatenate([np.zeros(1, np.int64), keys]))[1:]      # unaligned key column: scalar path
    vb = dev(np.concatenate([np.zeros(3, np.int64), v]))[3:]
    got_k, got, _ = ocl.select_group_aggregate([], [base], [vb], C3_AGGS, key_sorted=True)
    rk, routs = oracle.sga([], [keys], [v], C3_AGGS, order_by_key=True)
    assert np.array_equal(got_k.cpu().numpy(), rk)
    assert all(np.array_equal(g.cpu().numpy(), r) for g, r in zip(got, routs))
    bad = keys.copy()
    bad[50000] = bad[50000] - 5                                         # not sorted
    with pytest.raises(ocl.OcelotError, match="INVALID_ARG"):
        ocl.select_group_aggregate([], [dev(bad)], [dev(v)], C3_AGGS, key_sorted=True)
    # output capacity too small -> the binding's restart grows it
    _check_sorted([], [keys], [v], C3_AGGS, out_capacity=10)


@pytest.mark.parametrize("mode", ["sorted", "tier6"])
def test_sorted_partials_merge(mode):
    """Multi-GPU pieces for the sort-based paths: row shards (runs cut at shard boundaries) -> partial
    rows (ocl_sga_partial) -> merge == oracle over all rows (fake exchange on one GPU)."""
    from paper_journals_pvldb_heimelspmm13_b200.distributed import shard_range
    n, P = 300001, 3
    li = datagen.lineitem_host(n, datagen.BASE_SEED + 3, shuffled=(mode == "tier6"))
    aggs = C3_AGGS + [{"op": "avg", "a": 0}]
    kw = dict(key_sorted=True) if mode == "sorted" else dict(tier=6)
    cap = n // 2
    parts, counts = [], []
    for r in range(P):
        s0, ln = shard_range(n, r, P)
        call = ocl.SgaCall([], [dev(li["orderkey"][s0:s0 + ln])], [dev(li["quantity"][s0:s0 + ln])], aggs,
                           expected_groups=cap, out_capacity=cap, **kw)
        part, cnt = ocl.sga_partial(call, cap)
        parts.append(part)
        counts.append(cnt)
    allp = torch.stack(parts).contiguous()
    call = ocl.SgaCall([], [dev(li["orderkey"])], [dev(li["quantity"])], aggs, expected_groups=cap, out_capacity=cap)
    ocl.merge_partials(call, allp, torch.cat(counts), P, cap)
    keys, outs = call.result()
    rk, routs = oracle.sga([], [li["orderkey"]], [li["quantity"]], aggs)
    dts = [np.int64]
    assert_results_equal(by_key(keys.cpu().numpy(), [o.cpu().numpy() for o in outs], aggs, dts),
                         by_key(rk, routs, aggs, dts), aggs, dts)
