"""CUDA path (through the C ABI) vs the CPU oracle, element by element.

Rules (BASELINE.json north_star): bitmaps / oids / integer
aggregates / MIN / MAX bit-exact; gids compared as a partition (canonicalised by
first occurrence) with keys_out a bijection onto the distinct qualifying keys;
fp64 SUM / AVG within 1e-9 relative per group.
"""
import numpy as np
import pytest
import torch

import datagen
import oracle
from tests._common import Q1_AGGS, Q1_PRED, assert_results_equal, by_key, canon_gids

pytestmark = pytest.mark.gpu

ocl = pytest.importorskip("paper_journals_pvldb_heimelspmm13_b200")
DEV = torch.device("cuda", 0)
SIZES = [0, 1, 31, 32, 33, 1023, 1024, 1025, 4097, 65536 + 17, (1 << 20) + 17]
TDT = {np.uint8: torch.uint8, np.int32: torch.int32, np.int64: torch.int64, np.float64: torch.float64}


def dev(a):
    return torch.from_numpy(np.ascontiguousarray(a)).to(DEV)


def host_u32(t):
    return t.cpu().numpy().view(np.uint32)


def rand_col(rng, dtype, n):
    if dtype == np.float64:
        return rng.integers(-1000, 1000, n).astype(np.float64) / 8.0
    if dtype == np.uint8:
        return rng.integers(0, 256, n).astype(np.uint8)
    return rng.integers(-1000, 1000, n).astype(dtype)


SPECS = [{}, {"lo": -10, "hi": 300}, {"lo": -10, "hi": 300, "lo_incl": False, "hi_incl": False},
         {"hi": 0, "anti": True}, {"lo": 5, "hi": 5}, {"lo": 50, "hi": -50}, {"lo": 17}]


# ---------------------------------------------------------------- a1
@pytest.mark.parametrize("dtype", [np.uint8, np.int32, np.int64, np.float64])
@pytest.mark.parametrize("n", SIZES)
def test_select_bitmap(dtype, n):
    rng = np.random.default_rng(n + 7)
    col = rand_col(rng, dtype, n)
    tcol = dev(col)
    for spec in SPECS:
        ref = oracle.select(col, spec)
        got = ocl.select_bitmap(tcol, spec)
        torch.cuda.synchronize()
        assert np.array_equal(host_u32(got), ref), (spec, n)


@pytest.mark.parametrize("offset", [1, 2, 3])
def test_select_bitmap_unaligned(offset):
    rng = np.random.default_rng(offset)
    n = 5000
    base = dev(rand_col(rng, np.int32, n + offset))
    col = base[offset:]
    spec = {"lo": -100, "hi": 400}
    ref = oracle.select(col.cpu().numpy(), spec)
    assert np.array_equal(host_u32(ocl.select_bitmap(col, spec)), ref)


def test_bitmap_combine():
    rng = np.random.default_rng(1)
    for n in [1, 33, 4097, 100003]:
        x = rng.integers(0, 10, n).astype(np.int32)
        a, b = oracle.select(x, {"hi": 5}), oracle.select(x, {"lo": 3})
        for op in ("and", "or", "andnot"):
            got = ocl.bitmap_combine(op, dev(a.view(np.int32)), dev(b.view(np.int32)), n)
            assert np.array_equal(host_u32(got), oracle.bitmap_combine(op, a, b, n)), (op, n)


# ---------------------------------------------------------------- a2 / a3
@pytest.mark.parametrize("n", SIZES + [3 * 65536 * 8 + 5])
@pytest.mark.parametrize("sel", [0.0, 0.013, 0.5, 1.0])
def test_prefix_compact(n, sel):
    rng = np.random.default_rng(n)
    p = (rng.random(n) < sel).astype(np.int32) if n else np.zeros(0, np.int32)
    bm = oracle.select(p, {"lo": 1})
    ref = oracle.compact(bm, n)
    oids, m = ocl.prefix_compact(dev(bm.view(np.int32)) if n else torch.zeros(1, dtype=torch.int32, device=DEV), n)
    mm = int(m.item())
    assert mm == len(ref)
    assert np.array_equal(oids[:mm].cpu().numpy().view(np.uint32), ref)


def test_gather():
    rng = np.random.default_rng(3)
    for dtype in (np.uint8, np.int32, np.int64, np.float64):
        col = rand_col(rng, dtype, 10000)
        oids = np.sort(rng.choice(10000, 3000, replace=False)).astype(np.uint32)
        got = ocl.gather(dev(col), dev(oids.view(np.int32)))
        assert np.array_equal(got.cpu().numpy(), oracle.gather(col, oids))


# ---------------------------------------------------------------- a4-a6
@pytest.mark.parametrize("kind,G", [("u8u8", 6), ("i64", 1000), ("i64", 200000), ("i32", 50), ("u8", 256),
                                    ("i32i32", 500), ("u8i32", 300), ("i64neg1", 10)])
@pytest.mark.parametrize("scheme", ["b200", "paper"])
def test_group_build(kind, G, scheme):
    rng = np.random.default_rng(G)
    n = 300000
    if kind == "u8u8":
        keys = [rng.choice(np.array([65, 78, 82], np.uint8), n), rng.choice(np.array([70, 79], np.uint8), n)]
    elif kind == "i64":
        keys = [(rng.integers(0, G, n) * 7919 - 5).astype(np.int64)]
    elif kind == "i32":
        keys = [rng.integers(-G // 2, G // 2, n).astype(np.int32)]
    elif kind == "i32i32":
        keys = [rng.integers(-G // 2, G // 2, n).astype(np.int32), rng.integers(-3, 3, n).astype(np.int32)]
    elif kind == "u8i32":   # mixed widths: the runtime-described key path
        keys = [rng.integers(0, 3, n).astype(np.uint8), rng.integers(-G // 6, G // 6, n).astype(np.int32)]
    elif kind == "i64neg1":  # key ~0 (all bits set) lives in the table's side entry
        keys = [rng.integers(-G // 2, G // 2, n).astype(np.int64)]
    else:
        keys = [rng.integers(0, 256, n).astype(np.uint8)]
    oids = np.flatnonzero(rng.random(n) < 0.7).astype(np.uint32)
    ref_g, ref_k = oracle.group_hash(keys, oids)
    gids, kout, ng, st = ocl.group_build([dev(k) for k in keys], oids=dev(oids.view(np.int32)),
                                         expected_groups=max(len(ref_k), 16), scheme=scheme)
    torch.cuda.synchronize()
    assert int(st.item()) == 0
    Gg = int(ng.item())
    assert Gg == len(ref_k)
    g = gids[:len(oids)].cpu().numpy()
    assert np.array_equal(canon_gids(g), canon_gids(ref_g))                  # same partition
    kk = kout[:Gg].cpu().numpy()
    assert sorted(kk.view(np.uint64).tolist()) == sorted(ref_k.view(np.uint64).tolist())   # bijection
    # gid -> key consistent with the first-occurrence oracle labels
    first = {}
    for j, gg in enumerate(g.tolist()):
        first.setdefault(gg, j)
    for gg, j in first.items():
        assert kk[gg] == ref_k[ref_g[j]]


@pytest.mark.parametrize("scheme", ["b200", "paper"])
def test_group_build_capacity_status(scheme):
    n = 5000
    keys = [np.arange(n, dtype=np.int64)]
    gids, kout, ng, st = ocl.group_build([dev(keys[0])], expected_groups=8, scheme=scheme)
    torch.cuda.synchronize()
    assert int(st.item()) == ocl.OCL_ERR_CAPACITY                            # restart signal


# ---------------------------------------------------------------- a7-a8
@pytest.mark.parametrize("G", [1, 4, 100, 5000, 300000])
def test_group_aggregate(G):
    rng = np.random.default_rng(G)
    n = 400000
    gids = rng.integers(0, G, n).astype(np.int32)
    v = rng.integers(-10**12, 10**12, n).astype(np.int64)
    d = rng.integers(0, 11, n).astype(np.int64)
    t = rng.integers(0, 9, n).astype(np.int64)
    f = rng.integers(0, 10**6, n).astype(np.float64) / 100.0
    vals = [v, d, t, f]
    aggs = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "min", "a": 0}, {"op": "max", "a": 0},
            {"op": "sum", "expr": "mul_1minus_1plus", "a": 0, "b": 1, "c": 2, "scale": 2},
            {"op": "avg", "a": 0}, {"op": "sum", "a": 3}, {"op": "min", "a": 3}, {"op": "max", "a": 3},
            {"op": "avg", "a": 3}]
    oids = np.flatnonzero(rng.random(n) < 0.6).astype(np.uint32)
    sub = gids[oids]
    ref = oracle.aggregate(sub, G, vals, aggs, oids=oids)
    got = ocl.group_aggregate(dev(sub), None, G, [dev(x) for x in vals], aggs, oids=dev(oids.view(np.int32)))
    keys = np.arange(G, dtype=np.int64)
    dts = [x.dtype for x in vals]
    g = by_key(keys, [o[:G].cpu().numpy() for o in got], aggs, dts)
    r = by_key(keys, ref, aggs, dts)
    # groups with no rows: COUNT 0 and SUM 0; MIN/MAX/AVG are SQL NULL (unspecified) -> compared only when present
    present = np.bincount(sub, minlength=G) > 0
    for k in np.flatnonzero(~present).tolist():
        assert g[k][0] == 0 and g[k][1] == 0
        del g[k], r[k]
    assert_results_equal(g, r, aggs, dts)


# ---------------------------------------------------------------- a9 fused
def _lineitem(n, seed, f64=False, shuffled=False):
    fields = datagen.LINEITEM_INT_FIELDS + (datagen.LINEITEM_F64_FIELDS if f64 else ())
    return datagen.lineitem_host(n, seed, fields=fields, shuffled=shuffled)


def ran_kernel():
    """Name of the fused kernel the last fused call on cuda:0 launched (ocl_ctx_last_kernel)."""
    return ocl.last_kernel(ocl.context(DEV))


def _check_sga(preds, keys, vals, aggs, expected_groups=4, tier=0, order_by_key=False, bitmap=False, rtol=1e-9,
               kernel=None, out_capacity=None):
    """Fused call vs oracle.sga; kernel (substring) asserts which fused kernel ran, so a dispatch change
    cannot silently move a test away from the kernel it is meant to cover."""
    k, outs, bm = ocl.select_group_aggregate([(dev(c), s) for c, s in preds], [dev(c) for c in keys],
                                             [dev(c) for c in vals], aggs, expected_groups=expected_groups,
                                             tier=tier, order_by_key=order_by_key, bitmap=bitmap,
                                             out_capacity=out_capacity)
    if kernel is not None:
        assert kernel in ran_kernel(), (kernel, ran_kernel())
    rk, routs = oracle.sga(preds, keys, vals, aggs, order_by_key=order_by_key)
    dts = [c.dtype for c in vals]
    assert_results_equal(by_key(k.cpu().numpy(), [o.cpu().numpy() for o in outs], aggs, dts),
                         by_key(rk, routs, aggs, dts), aggs, dts, rtol=rtol)
    if order_by_key:
        assert k.cpu().numpy().tolist() == rk.tolist()
    if bitmap:
        n = len((preds[0][0] if preds else keys[0]))
        ref = np.full((n + 31) // 32, 0xFFFFFFFF, np.uint32)
        for c, s in preds:
            ref &= oracle.select(c, s)
        if n % 32:
            ref[-1] &= (1 << (n % 32)) - 1
        assert np.array_equal(host_u32(bm), ref)
    return k, outs


def _q1(li, f64=False):
    if f64:
        vals = [li["quantity_f"], li["extendedprice_f"], li["discount_f"], li["tax_f"]]
        aggs = [dict(a, scale=0) for a in Q1_AGGS]
    else:
        vals = [li["quantity"], li["extendedprice"], li["discount"], li["tax"]]
        aggs = Q1_AGGS
    return [(li["shipdate"], Q1_PRED)], [li["returnflag"], li["linestatus"]], vals, aggs


@pytest.mark.parametrize("tier", [1, 2])
@pytest.mark.parametrize("n", [1, 127, 128, 60000, 1000003])
def test_fused_q1_int(tier, n):
    li = _lineitem(n, datagen.BASE_SEED + 1)
    p, k, v, a = _q1(li)
    # tier 1: the Q1 + MIN/MAX signature kernel (the MIN/MAX pair matches it) when n fills a pipeline stage
    want = ("k_sga_bulk<Sig Q1+MINMAX int64>" if n >= 512 else "k_sga<DynShape>") if tier == 1 else "k_sga_glb"
    _check_sga(p, k, v, a + [{"op": "sum", "a": 2}, {"op": "min", "a": 0}, {"op": "max", "a": 1}], tier=tier,
               order_by_key=True, bitmap=True, kernel=want)


@pytest.mark.parametrize("tier", [1, 2])
def test_fused_q1_f64(tier):
    li = _lineitem(6000000 if tier == 1 else 300000, datagen.BASE_SEED + 2, f64=True)
    p, k, v, a = _q1(li, f64=True)
    _check_sga(p, k, v, a + [{"op": "min", "a": 0}, {"op": "max", "a": 1}], tier=tier,
               kernel="k_sga_bulk<Sig Q1+MINMAX fp64>" if tier == 1 else "k_sga_glb")


def test_fused_worked_example():
    from tests._common import golden_columns, load_golden
    c = golden_columns(load_golden())
    li = dict(c)
    p, k, v, a = _q1(li)
    _check_sga(p, k, v, a, order_by_key=True, bitmap=True, rtol=0.0, kernel="k_sga_priv<Sig Q1 int64>")


@pytest.mark.parametrize("G", [3, 5, 64, 5000, 200000])
def test_fused_many_groups(G):
    """Register tier overflows (G > 4 slots) and global tier; both exact."""
    n = 500000
    sw = datagen.sweep_host(n, datagen.BASE_SEED + 5, G, s=1.0)
    preds = [(sw["p"], {"hi": 499999})]
    aggs = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "min", "a": 0}, {"op": "max", "a": 0},
            {"op": "avg", "a": 0}]
    for tier in (0, 1, 2, 3, 4, 5):
        _check_sga(preds, [sw["key"]], [sw["v"]], aggs, expected_groups=G, tier=tier)


@pytest.mark.parametrize("G,s,sel", [(16, 0.0, 10**6), (256, 1.5, 5 * 10**5), (4096, 1.0, 10**4), (1 << 16, 1.5, 10**6),
                                     (1 << 20, 0.0, 5 * 10**5)])
def test_fused_sweep_c5_shape(G, s, sel):
    """C5 sweep points (scaled to 2^21 rows): count, sum, min, max of v (+ fp64 sum/avg of v/100), auto tier."""
    n = 1 << 21
    sw = datagen.sweep_host(n, datagen.BASE_SEED + 5, G, s=s, f64=True)
    preds = [(sw["p"], {"hi": sel - 1})]
    aggs = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "min", "a": 0}, {"op": "max", "a": 0},
            {"op": "sum", "a": 1}, {"op": "avg", "a": 1}]
    _check_sga(preds, [sw["key"]], [sw["v"], sw["v_f"]], aggs, expected_groups=G)


def test_fused_edge_cases():
    rng = np.random.default_rng(5)
    n = 10000
    x = rng.integers(0, 100, n).astype(np.int64)
    # empty selection
    k, outs = _check_sga([(x, {"lo": 1000})], [x], [x], [{"op": "count"}, {"op": "sum", "a": 0}])
    assert len(k) == 0
    # no predicate, no keys: one group
    _check_sga([], [], [x], [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "avg", "a": 0}])
    # key == ~0 (the table's reserved pattern) and key 0
    kk = np.where(x < 30, -1, np.where(x < 60, 0, 5)).astype(np.int64)
    _check_sga([(x, {"hi": 90})], [kk], [x], [{"op": "count"}, {"op": "sum", "a": 0}], tier=1)
    _check_sga([(x, {"hi": 90})], [kk], [x], [{"op": "count"}, {"op": "max", "a": 0}], tier=2)
    # int128: sums beyond int64 and factors beyond int32 (slow exact path)
    big = np.full(n, 2**62 + 3, np.int64)
    big[::7] = -(2**63)
    _check_sga([], [x % 3], [big, x], [{"op": "sum", "a": 0}, {"op": "avg", "a": 0},
                                        {"op": "sum", "expr": "mul_1minus", "a": 0, "b": 1, "scale": 2},
                                        {"op": "sum", "expr": "mul_1minus_1plus", "a": 0, "b": 1, "c": 1,
                                         "scale": 3}], tier=1)
    # mixed int / fp64 value columns
    f = x.astype(np.float64) / 3.0
    _check_sga([(x, {"lo": 10})], [x % 4], [x, f], [{"op": "sum", "a": 0}, {"op": "sum", "a": 1},
                                                    {"op": "min", "a": 1}, {"op": "avg", "a": 1}])
    # two i32 keys, f64 predicate, anti predicate, two predicates
    a32 = rng.integers(-3, 3, n).astype(np.int32)
    b32 = rng.integers(-2, 2, n).astype(np.int32)
    fp = rng.random(n)
    _check_sga([(fp, {"lo": 0.25, "lo_incl": False}), (x, {"lo": 20, "hi": 70, "anti": True})], [a32, b32], [x],
               [{"op": "count"}, {"op": "sum", "a": 0}], expected_groups=24, tier=2, bitmap=True)


@pytest.mark.parametrize("offset", [1, 3])
def test_fused_unaligned_columns(offset):
    """Device columns that start `offset` elements into their allocation (torch slices keep the offset, so
    u8 / i32 / i64 columns are 1- / 4- / 8-byte but not 16-byte aligned): the scalar-load path."""
    n = 20000
    li = _lineitem(n + offset, 11)
    p, k, v, a = _q1(li)
    sl = lambda c: dev(c)[offset:]
    assert sl(li["quantity"]).data_ptr() % 16 != 0
    keys, outs, bm = ocl.select_group_aggregate([(sl(c), s) for c, s in p], [sl(c) for c in k], [sl(c) for c in v],
                                                a, expected_groups=4, tier=1, order_by_key=True, bitmap=True)
    assert "k_sga<DynShape>" in ran_kernel()                 # unaligned: no vector loads, no copy engine
    p0 = [(c[offset:], s) for c, s in p]
    k0, v0 = [c[offset:] for c in k], [c[offset:] for c in v]
    rk, routs = oracle.sga(p0, k0, v0, a, order_by_key=True)
    dts = [c.dtype for c in v0]
    assert keys.cpu().numpy().tolist() == rk.tolist()
    assert_results_equal(by_key(keys.cpu().numpy(), [o.cpu().numpy() for o in outs], a, dts),
                         by_key(rk, routs, a, dts), a, dts)
    assert np.array_equal(host_u32(bm), oracle.select(p0[0][0], p0[0][1]))


def test_fused_c3_orderkey():
    """C3 shape (scaled down): GROUP BY orderkey, ~n/4 groups, HBM-resident table, both layouts."""
    n = 400000
    for shuffled in (False, True):
        li = _lineitem(n, datagen.BASE_SEED + 3, shuffled=shuffled)
        aggs = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "min", "a": 0}, {"op": "max", "a": 0}]
        for tier in (2, 5):
            _check_sga([], [li["orderkey"]], [li["quantity"]], aggs, expected_groups=n // 4, tier=tier,
                       kernel="k_sga_glb" if tier == 2 else "hash-partitioned")


@pytest.mark.parametrize("n", [1, 1000, 70001, 1 << 20])
def test_fused_partitioned_edges(n):
    """Hash-partitioned tier (tier 5): ragged sizes, the key ~0, values outside int32 (exact
    per-row path), several value columns (32-byte records), two keys, a partition holding
    most rows (heavy hitter), more groups than expected (shared-table overflow)."""
    rng = np.random.default_rng(n)
    x = rng.integers(-1000, 1000, n).astype(np.int64)
    key = rng.integers(0, max(1, n // 3), n).astype(np.int64)
    key[::11] = -1                                       # ~0: the side entry
    key[rng.random(n) < 0.4] = 7                         # heavy hitter
    big = x.copy()
    big[::13] = 2**40 + 5                                # outside int32: exact per-row path
    aggs = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "min", "a": 0}, {"op": "max", "a": 0},
            {"op": "sum", "a": 1}, {"op": "min", "a": 2}, {"op": "max", "a": 2}, {"op": "avg", "a": 1}]
    for G in (n // 3 + 2, 8):
        _check_sga([(x, {"lo": -900})], [key], [x, big, x // 7], aggs, expected_groups=G, tier=5)
    k32 = (x % 5).astype(np.int32)
    _check_sga([], [(key & 0x7FFFFFFF).astype(np.int32), k32], [x], [{"op": "count"}, {"op": "sum", "a": 0}], expected_groups=max(8, n // 2), tier=5)
    _check_sga([(x, {"lo": 5000})], [key], [x], [{"op": "count"}], expected_groups=n + 8, tier=5)   # empty


@pytest.mark.parametrize("n,scatter", [(1 << 20, None), (1 << 20, "0"), (1 << 20, "1"), (1 << 20, "2"), (1 << 20, "3"), (1 << 23, None), (1 << 23, "1")])
def test_fused_partitioned_near_full(n, scatter, monkeypatch):
    """Tier 5 with ~1.8x the expected groups: 128 partitions of ~1840 keys in 2048-slot shared tables, so
    probe sequences pass the shared table's limit and partitions overflow into their HBM region.  At 2^20
    rows every partition is one work item (the lazily zeroed region is cleared by the overflowing CTA);
    at 2^23 partitions are split over work items (regions cleared before pass 1b).  Every pass-1b
    scatter mode (OCL_PSCAT: 0 one-level per-row claims, 1 tiled, 2 / 3 one-level without prefetch, 4 / 8 rows)."""
    if scatter is not None:
        monkeypatch.setenv("OCL_PSCAT", scatter)
    rng = np.random.default_rng(n + 17)
    E = 1 << 17
    key = rng.integers(0, int(1.8 * E), n).astype(np.int64) * 7919
    x = rng.integers(-10**6, 10**6, n).astype(np.int64)
    aggs = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "min", "a": 0}, {"op": "max", "a": 0}]
    _check_sga([], [key], [x], aggs, expected_groups=E, tier=5, out_capacity=4 * E, kernel="hash-partitioned")


@pytest.mark.parametrize("G", [5000, 300000])
def test_fused_partitioned_sparse(G):
    """Tier 5 at ~2 % selectivity: the device-side sample picks the sparse mode (count pass lists the
    qualifying rows per block, the level-1 scatter reads those lists); one level (G = 5000) and two
    levels (G = 300000); qualifying rows include values outside int32 and the key ~0 (exact path)."""
    n = 1 << 21
    rng = np.random.default_rng(G)
    pcol = rng.integers(0, 1000, n).astype(np.int32)
    key = rng.integers(0, G, n).astype(np.int64) * 2654435761
    key[::997] = -1
    x = rng.integers(-10**6, 10**6, n).astype(np.int64)
    x[::1301] = 2**40 + 7
    aggs = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "min", "a": 0}, {"op": "max", "a": 0}]
    _check_sga([(pcol, {"hi": 19})], [key], [x], aggs, expected_groups=G, tier=5, kernel="hash-partitioned")


@pytest.mark.parametrize("n,G", [(1 << 22, 4096), (1 << 23, 1 << 16)])
def test_fused_partitioned_small_partitions(n, G):
    """Many rows per key: partitions are split into several pass-2 items anyway, so the tier targets 256
    (G = 4096: 16 partitions) or 512 (G = 2^16: 128, one scatter level) keys per partition instead of
    1024; the HBM table then no longer has kPartCap slots per partition (no direct emission)."""
    rng = np.random.default_rng(G + 3)
    key = rng.integers(0, G, n).astype(np.int64) * 1000003 - 77
    x = rng.integers(-10**6, 10**6, n).astype(np.int64)
    aggs = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "min", "a": 0}, {"op": "max", "a": 0},
            {"op": "avg", "a": 0}]
    _check_sga([], [key], [x], aggs, expected_groups=G, tier=5, kernel="hash-partitioned")


def test_fused_capacity_retry():
    n = 50000
    x = np.arange(n, dtype=np.int64)
    # expected_groups far too small: the binding restarts with a larger table
    _check_sga([], [x], [x], [{"op": "count"}, {"op": "sum", "a": 0}], expected_groups=4, tier=2)


# ---------------------------------------------------------------- host buffers (e2e path)
def test_host_path_matches():
    n = 3 * (1 << 16) + 123
    li = _lineitem(n, 17)
    p, k, v, a = _q1(li)
    t = lambda c: torch.from_numpy(c).pin_memory()
    keys, outs = ocl.select_group_aggregate_host([(t(c), s) for c, s in p], [t(c) for c in k], [t(c) for c in v], a,
                                                 expected_groups=4, order_by_key=True, chunk_rows=1 << 16)
    rk, routs = oracle.sga(p, k, v, a, order_by_key=True)
    dts = [c.dtype for c in v]
    assert_results_equal(by_key(keys.numpy(), [o.numpy() for o in outs], a, dts), by_key(rk, routs, a, dts), a, dts)


# ---------------------------------------------------------------- multi-GPU merge (fake exchange)
@pytest.mark.parametrize("P", [2, 3, 8])
def test_sharded_partials_merge(P):
    """Row shards -> partial tables -> concatenated (stand-in for the allgather) -> merge == oracle on all rows."""
    from paper_journals_pvldb_heimelspmm13_b200.distributed import shard_range
    n = 250001
    li = _lineitem(n, datagen.BASE_SEED + 4)
    p, k, v, a = _q1(li)
    a = a + [{"op": "min", "a": 0}, {"op": "max", "a": 1}]
    cap = 16
    parts, counts = [], []
    for r in range(P):
        s0, ln = shard_range(n, r, P)
        call = ocl.SgaCall([(dev(c[s0:s0 + ln]), s) for c, s in p], [dev(c[s0:s0 + ln]) for c in k],
                           [dev(c[s0:s0 + ln]) for c in v], a, expected_groups=4, out_capacity=cap)
        part, cnt = ocl.sga_partial(call, cap)
        parts.append(part)
        counts.append(cnt)
    allp = torch.stack(parts).contiguous()
    allc = torch.cat(counts)
    call = ocl.SgaCall([(dev(c), s) for c, s in p], [dev(c) for c in k], [dev(c) for c in v], a,
                       expected_groups=4, out_capacity=cap, order_by_key=True)
    ocl.merge_partials(call, allp, allc, P, cap)
    keys, outs = call.result()
    rk, routs = oracle.sga(p, k, v, a, order_by_key=True)
    dts = [c.dtype for c in v]
    assert keys.cpu().numpy().tolist() == rk.tolist()
    assert_results_equal(by_key(keys.cpu().numpy(), [o.cpu().numpy() for o in outs], a, dts),
                         by_key(rk, routs, a, dts), a, dts)


def test_device_generator_matches_host():
    n = 100003
    h = datagen.lineitem_host(n, 99, fields=datagen.LINEITEM_INT_FIELDS + datagen.LINEITEM_F64_FIELDS,
                              row0=5000, n_total=10**6)
    d = datagen.lineitem_device(n, 99, fields=datagen.LINEITEM_INT_FIELDS + datagen.LINEITEM_F64_FIELDS,
                                row0=5000, n_total=10**6)
    for f in h:
        assert np.array_equal(d[f].cpu().numpy(), h[f]), f
    sh = datagen.sweep_host(n, 7, 1 << 12, s=1.5, f64=True)
    sd = datagen.sweep_device(n, 7, 1 << 12, s=1.5, f64=True)
    for f in sh:
        assert np.array_equal(sd[f].cpu().numpy(), sh[f]), f


def test_fused_q1_unified_static_shape(monkeypatch):
    """The unified kernel's static Q1 shape (OCL_NO_SPEC=1 bypasses the hand-specialised Q1 kernel)."""
    monkeypatch.setenv("OCL_NO_SPEC", "1")
    for n in (1000, 300001):
        li = _lineitem(n, datagen.BASE_SEED + 1)
        p, k, v, a = _q1(li)
        _check_sga(p, k, v, a, tier=1, order_by_key=True, bitmap=True, kernel="k_sga<StaticShape Q1 int64>")
        lf = _lineitem(n, datagen.BASE_SEED + 2, f64=True)
        p, k, v, a = _q1(lf, f64=True)
        _check_sga(p, k, v, a, tier=1, kernel="k_sga<StaticShape Q1 fp64>")


# ---------------------------------------------------------------- NEXT-2: hash-routed all-to-all merge (fake exchange)
@pytest.mark.parametrize("P,G", [(2, 5000), (3, 40000), (8, 200000)])
def test_routed_alltoall_merge(P, G):
    """Shards -> partial tables -> ocl_route_partials -> destination d gets block d of every shard
    (stand-in for all_to_all) -> merge per destination: every key at its owner, union == oracle."""
    from paper_journals_pvldb_heimelspmm13_b200.distributed import shard_range
    from tests.test_distributed_cpu import route_of
    rng = np.random.default_rng(G)
    n = 600000
    keys = (rng.integers(0, G, n) * 2654435761 % (1 << 40)).astype(np.int64)
    v = rng.integers(-10**6, 10**6, n).astype(np.int64)
    f = rng.integers(0, 10**6, n).astype(np.float64) / 100.0
    aggs = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "min", "a": 0}, {"op": "max", "a": 0},
            {"op": "avg", "a": 1}, {"op": "sum", "a": 1}]
    cap = 2 * G
    blocks = [[] for _ in range(P)]
    for r in range(P):
        s0, ln = shard_range(n, r, P)
        call = ocl.SgaCall([], [dev(keys[s0:s0 + ln])], [dev(v[s0:s0 + ln]), dev(f[s0:s0 + ln])], aggs,
                           expected_groups=G, out_capacity=cap)
        part, cnt = ocl.sga_partial(call, cap)
        routed, counts = ocl.route_partials(part, cnt, P)
        c = counts.cpu().numpy()
        assert c.sum() == int(cnt.item())
        off = np.concatenate([[0], np.cumsum(c)])
        for d in range(P):
            blocks[d].append(routed[off[d]:off[d + 1]])
    got_k, got_o = [], []
    for d in range(P):
        recv = torch.cat(blocks[d]).contiguous()
        call = ocl.SgaCall([], [dev(keys)], [dev(v), dev(f)], aggs, expected_groups=G, out_capacity=cap)
        total = recv.shape[0]
        ocl.merge_partials(call, recv if total else torch.zeros((1, recv.shape[1]), dtype=torch.uint8, device=DEV),
                           torch.tensor([total], dtype=torch.int64, device=DEV), 1, max(total, 1))
        k, o = call.result()
        k = k.cpu().numpy()
        assert (route_of(k.view(np.uint64), P).astype(np.int64) == d).all()   # partition d only
        got_k.append(k)
        got_o.append([x.cpu().numpy() for x in o])
    gk = np.concatenate(got_k)
    go = [np.concatenate([g[i] for g in got_o]) for i in range(len(aggs))]
    rk, routs = oracle.sga([], [keys], [v, f], aggs)
    dts = [v.dtype, f.dtype]
    assert_results_equal(by_key(gk, go, aggs, dts), by_key(rk, routs, aggs, dts), aggs, dts)


def test_cuda_graph_replay():
    """SgaCall.capture(): the whole fused call (table init, kernel, finalisation) replayed as one CUDA graph
    gives the oracle's result, repeatedly (C1 shape, and the sorted path)."""
    li = _lineitem(60000, datagen.BASE_SEED + 1)
    p, k, v, a = _q1(li)
    call = ocl.SgaCall([(dev(c), s) for c, s in p], [dev(c) for c in k], [dev(c) for c in v], a,
                       expected_groups=4, order_by_key=True)
    g = call.capture()
    rk, routs = oracle.sga(p, k, v, a, order_by_key=True)
    dts = [c.dtype for c in v]
    for _ in range(3):
        call.outs[0].zero_()
        g.replay()
        keys, outs = call.result()
        assert keys.cpu().numpy().tolist() == rk.tolist()
        assert_results_equal(by_key(keys.cpu().numpy(), [o.cpu().numpy() for o in outs], a, dts),
                             by_key(rk, routs, a, dts), a, dts)
    aggs = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "min", "a": 0}, {"op": "max", "a": 0}]
    call = ocl.SgaCall([], [dev(li["orderkey"])], [dev(li["quantity"])], aggs, expected_groups=20000,
                       out_capacity=20000, key_sorted=True)
    g = call.capture()
    g.replay()
    keys, outs = call.result()
    rk, routs = oracle.sga([], [li["orderkey"]], [li["quantity"]], aggs, order_by_key=True)
    assert np.array_equal(keys.cpu().numpy(), rk)
    assert all(np.array_equal(o.cpu().numpy(), r) for o, r in zip(outs, routs))


@pytest.mark.parametrize("G", [50000, 1 << 20])
def test_partitioned_partials_merge(G):
    """Partial rows from the hash-partitioned tier (tier 5: rows emitted straight from shared memory as
    partial rows, dirty partitions from the HBM table) -> merge == oracle; values beyond int32 and the
    key ~0 force exact-path (dirty) partitions."""
    from paper_journals_pvldb_heimelspmm13_b200.distributed import shard_range
    rng = np.random.default_rng(G)
    n, P = (1 << 21) + 3, 2
    keys = rng.integers(0, G, n).astype(np.int64) * 2654435761 % (1 << 40)
    keys[::4099] = -1                                                   # key ~0
    v = rng.integers(-10**6, 10**6, n).astype(np.int64)
    v[::10007] = 1 << 40                                                # beyond int32: exact path
    aggs = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "min", "a": 0}, {"op": "max", "a": 0}]
    cap = 2 * G + 16
    parts, counts = [], []
    for r in range(P):
        s0, ln = shard_range(n, r, P)
        call = ocl.SgaCall([], [dev(keys[s0:s0 + ln])], [dev(v[s0:s0 + ln])], aggs, expected_groups=G,
                           out_capacity=cap, tier=5)
        part, cnt = ocl.sga_partial(call, cap)
        parts.append(part)
        counts.append(cnt)
    call = ocl.SgaCall([], [dev(keys)], [dev(v)], aggs, expected_groups=G, out_capacity=cap)
    ocl.merge_partials(call, torch.stack(parts).contiguous(), torch.cat(counts), P, cap)
    k, outs = call.result()
    rk, routs = oracle.sga([], [keys], [v], aggs)
    dts = [np.int64]
    assert_results_equal(by_key(k.cpu().numpy(), [o.cpu().numpy() for o in outs], aggs, dts),
                         by_key(rk, routs, aggs, dts), aggs, dts)
