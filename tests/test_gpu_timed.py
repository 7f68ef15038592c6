"""Parity of the exact kernels the benchmark times ("close the parity gaps").

The C1 / C2 / C4 numbers come from the Q1-signature kernels of fused_spec.cu:
``k_sga_bulk<Sig Q1 int64|fp64>`` (TMA bulk pipeline, default) and ``k_sga_priv<Sig ...>``
(register loads; ``OCL_BULK=0`` or fewer rows than one pipeline stage).  Each test here runs
the bench's own plan — the TPC-H Q1 aggregates with no MIN/MAX, so ``spec_match`` accepts it —
compares every group with the oracle (SURVEY §8(c) rules: integers bit-exact, fp64 SUM / AVG
within 1e-9 relative) and asserts the kernel that ran (``ocl_ctx_last_kernel``).

Covered: every bulk pipeline configuration (``OCL_BULK`` 1-7, read per launch), ragged sizes
around the stage size (n < R runs ``k_sga_priv``; n >= R the bulk kernel plus its scalar tail),
the bitmap output of the bulk kernel, and rows outside the int32 fast path (the exact
per-row int128 path inside the specialised kernels).  PAPER.md L562-568 (aggregation),
L429-438 (bitmap).
"""
import numpy as np
import pytest

import datagen
from tests._common import Q1_AGGS, Q1_AGGS_F64
from tests.test_gpu_parity import _check_sga, _lineitem, ran_kernel

pytestmark = pytest.mark.gpu

# OCL_BULK -> rows per pipeline stage (fused_spec.cu launch_bulk_cfg); None = default (int 7, fp64 3)
STAGE_ROWS = {None: 512, "0": 512, "1": 1024, "2": 512, "3": 512, "4": 512, "5": 256, "6": 256, "7": 512}


def _q1_plan(li, f64):
    if f64:
        vals = [li["quantity_f"], li["extendedprice_f"], li["discount_f"], li["tax_f"]]
        return [(li["shipdate"], {"hi": 10471})], [li["returnflag"], li["linestatus"]], vals, Q1_AGGS_F64
    vals = [li["quantity"], li["extendedprice"], li["discount"], li["tax"]]
    return [(li["shipdate"], {"hi": 10471})], [li["returnflag"], li["linestatus"]], vals, Q1_AGGS


def _expect(f64, n, cfg):
    sig = "fp64" if f64 else "int64"
    if cfg == "0" or n < STAGE_ROWS[cfg]:
        return f"k_sga_priv<Sig Q1 {sig}>"
    return f"k_sga_bulk<Sig Q1 {sig}>"


@pytest.mark.parametrize("n", [1, 100, 511, 512, 513, 1024 + 17, 4 * 512 * 148 + 333, 6_000_000])
def test_c2_kernel_fp64_q1(n):
    """C2's timed kernel: k_sga_bulk<SigQ1F> (default fp64 config <256, 512, 2>)."""
    li = _lineitem(n, datagen.BASE_SEED + 2, f64=True)
    p, k, v, a = _q1_plan(li, True)
    _check_sga(p, k, v, a, order_by_key=True, kernel=_expect(True, n, None))


@pytest.mark.parametrize("n", [1, 511, 512, 60_000, 1_000_003])
def test_c1_c4_kernel_int_q1(n):
    """C1 / C4's timed kernel: k_sga_bulk<SigQ1I> (default int config <128, 512, 2>)."""
    li = _lineitem(n, datagen.BASE_SEED + 4)
    p, k, v, a = _q1_plan(li, False)
    _check_sga(p, k, v, a, order_by_key=True, kernel=_expect(False, n, None))


@pytest.mark.parametrize("cfg", ["0", "1", "2", "3", "4", "5", "6", "7"])
@pytest.mark.parametrize("f64", [False, True])
def test_bulk_configs(monkeypatch, cfg, f64):
    """Every pipeline configuration (OCL_BULK, read per launch) on a size with several chunks per CTA and a
    ragged tail, plus one size below its stage.  Repeated: a stage-reuse race (the release of a stage before
    the warp's shared-memory loads had read it, fixed with mbar_release_reads in bulk.cuh) showed up as a
    few rows counted in the wrong group in some runs, most often with the 1-stage ring (cfg 4)."""
    monkeypatch.setenv("OCL_BULK", cfg)
    for n in (STAGE_ROWS[cfg] - 1, 3 * 148 * 2048 + 1000 + 17):   # cfg "0": k_sga_priv at both sizes
        li = _lineitem(n, datagen.BASE_SEED + 2 + (n & 7), f64=f64)
        p, k, v, a = _q1_plan(li, f64)
        for _ in range(3 if n > 100_000 else 1):
            _check_sga(p, k, v, a, order_by_key=True, kernel=_expect(f64, n, cfg))


@pytest.mark.parametrize("cfg", [None, "0", "5"])
@pytest.mark.parametrize("f64", [False, True])
def test_spec_bitmap_out(monkeypatch, cfg, f64):
    """bitmap_out emitted by the specialised kernels (bulk stages and the scalar tail), n >= R."""
    if cfg is not None:
        monkeypatch.setenv("OCL_BULK", cfg)
    n = 1_000_003
    li = _lineitem(n, datagen.BASE_SEED + 4, f64=f64)
    p, k, v, a = _q1_plan(li, f64)
    _check_sga(p, k, v, a, order_by_key=True, bitmap=True, kernel=_expect(f64, n, cfg))


@pytest.mark.parametrize("cfg", [None, "0"])
@pytest.mark.parametrize("n", [300, 700_001])
def test_spec_values_beyond_int32(monkeypatch, cfg, n):
    """Q1-signature plan whose rows leave the int32 fast path: quantities >= 2^31, prices whose products
    exceed 2^62, negative values; those rows take the exact int128 per-row update of the HBM entry
    (fused_spec.cu priv_slot -> update_entry_slow) while the rest stay in the private slots."""
    if cfg is not None:
        monkeypatch.setenv("OCL_BULK", cfg)
    li = _lineitem(n, datagen.BASE_SEED + 4)
    q, pr, d, t = (li[f].copy() for f in ("quantity", "extendedprice", "discount", "tax"))
    q[::97] = 3 * (1 << 40) + 1                     # COL value beyond int32
    pr[::101] = (1 << 35) + 7                       # product factor beyond int32
    pr[5::211] = (1 << 62) - 3                      # products beyond int64 (int128 accumulation)
    q[7::89] = -(1 << 33)                           # negative, beyond int32
    d[3::53] = -(1 << 31)                           # S - b beyond int32
    li.update(quantity=q, extendedprice=pr, discount=d, tax=t)
    p, k, v, a = _q1_plan(li, False)
    _check_sga(p, k, v, a, order_by_key=True, kernel=_expect(False, n, cfg))
    assert "Sig Q1 int64" in ran_kernel()


def test_spec_all_rows_filtered_and_one_group():
    """Degenerate Q1-signature inputs: every row filtered out (G = 0) and a single group."""
    n = 100_000
    li = _lineitem(n, datagen.BASE_SEED + 4)
    p, k, v, a = _q1_plan(li, False)
    keys, _ = _check_sga([(li["shipdate"], {"hi": 0})], k, v, a, order_by_key=True,
                         kernel="k_sga_bulk<Sig Q1 int64>")
    assert len(keys) == 0
    rf = np.full(n, ord("N"), np.uint8)
    ls = np.full(n, ord("O"), np.uint8)
    keys, _ = _check_sga(p, [rf, ls], v, a, order_by_key=True, kernel="k_sga_bulk<Sig Q1 int64>")
    assert keys.cpu().numpy().tolist() == [(ord("N") << 8) | ord("O")]


# ---------------------------------------------------------------- Q1 + MIN/MAX (bench workload c4mm)
Q1MM_EXTRA = [{"op": "min", "a": 0}, {"op": "max", "a": 1}]


@pytest.mark.parametrize("f64", [False, True])
@pytest.mark.parametrize("n", [255, 511, 512, 100_003, 3_000_017])
def test_c4mm_kernel(f64, n):
    """Q1 + MIN(quantity) + MAX(extendedprice): the signature kernel with MIN/MAX private fields
    (k_sga_bulk<Sig Q1+MINMAX>; int64 on a 256-row stage ring, fp64 on 512); smaller inputs fall back to
    the unified kernel."""
    li = _lineitem(n, datagen.BASE_SEED + 4, f64=f64)
    p, k, v, a = _q1_plan(li, f64)
    stage = 512 if f64 else 256
    want = f"k_sga_bulk<Sig Q1+MINMAX {'fp64' if f64 else 'int64'}>" if n >= stage else "k_sga<"
    _check_sga(p, k, v, a + Q1MM_EXTRA, order_by_key=True, kernel=want)


def test_c4mm_extremes():
    """MIN/MAX fields at the int32 range ends (encodings 0 and ~0) and beyond int32 (exact slow path)."""
    n = 200_000
    li = _lineitem(n, datagen.BASE_SEED + 4)
    q, pr = li["quantity"].copy(), li["extendedprice"].copy()
    q[::1001] = 2**31 - 1
    q[5::1003] = -(2**31)
    pr[7::997] = 2**31 - 1
    pr[9::991] = -(2**31)
    q[11::5003] = 2**40                                  # beyond int32: HBM entry, exact
    li.update(quantity=q, extendedprice=pr)
    p, k, v, a = _q1_plan(li, False)
    _check_sga(p, k, v, a + Q1MM_EXTRA, order_by_key=True, kernel="k_sga_bulk<Sig Q1+MINMAX int64>")


# ---------------------------------------------------------------- C5 / C3 group-by signatures
C5_AGGS = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "min", "a": 0}, {"op": "max", "a": 0}]


def _c5_tier(G):
    return "4 private slots" if G <= 4 else "CTA table"


@pytest.mark.parametrize("G", [4, 16, 32, 64, 256, 1024, 2048])
@pytest.mark.parametrize("zipf,sel", [(0.0, 10**6), (1.5, 5 * 10**5), (1.0, 10**4)])
def test_c5_signature_tiers(G, zipf, sel):
    """The C5 bench plan (WHERE p < T GROUP BY key: COUNT, SUM, MIN, MAX of v) on both accumulation tiers
    of k_sga_bulk<Sig pred i32, key i64> (private slots, CTA table), uniform
    and skewed keys (Zipf 1.5 puts ~38 % of the rows on one key), three selectivities."""
    n = (1 << 21) + 77
    sw = datagen.sweep_host(n, datagen.BASE_SEED + 5, G, s=zipf)
    preds = [(sw["p"], {"hi": sel - 1})]
    _check_sga(preds, [sw["key"]], [sw["v"]], C5_AGGS, expected_groups=G,
               kernel=f"k_sga_bulk<Sig pred i32, key i64, COUNT/SUM/MIN/MAX; {_c5_tier(G)}>")


@pytest.mark.parametrize("G", [4, 16, 32, 1000])
def test_c3_signature_tiers(G):
    """No predicate (C3 shape): GROUP BY key, COUNT / SUM / MIN / MAX."""
    n = 1_000_003
    sw = datagen.sweep_host(n, datagen.BASE_SEED + 3, G, s=0.5)
    _check_sga([], [sw["key"]], [sw["v"]], C5_AGGS, expected_groups=G,
               kernel=f"k_sga_bulk<Sig key i64, COUNT/SUM/MIN/MAX; {_c5_tier(G)}>")


@pytest.mark.parametrize("G,eg", [(40, 4), (100, 32), (3000, 2048), (3, 300)])
def test_signature_tier_overflow(G, eg):
    """More distinct keys than the tier holds (expected_groups underestimated): keys beyond the private
    slots / a full table replica take the exact HBM update; the result is still exact (the HBM table is sized
    by the restart of select_group_aggregate)."""
    n = 600_001
    rng = np.random.default_rng(G)
    key = ((rng.integers(0, G, n).astype(np.uint64) * np.uint64(0x9E3779B97F4A7C15)) >> np.uint64(2)).astype(np.int64)
    v = rng.integers(-10**6, 10**6, n).astype(np.int64)
    p = rng.integers(0, 100, n).astype(np.int32)
    _check_sga([(p, {"hi": 89})], [key], [v], C5_AGGS, expected_groups=eg,
               kernel="k_sga_bulk<Sig pred i32, key i64")


def test_signature_exact_paths():
    """C5 shape with values beyond int32 (exact int128 per-row path), the key ~0 (side entry), negative
    values and int32 extremes, on the private and CTA tiers."""
    n = 300_007
    rng = np.random.default_rng(9)
    for G in (8, 500):
        key = rng.integers(0, G, n).astype(np.int64) * 7919 - 3
        key[::97] = -1                                     # ~0
        v = rng.integers(-2**31, 2**31, n).astype(np.int64)
        v[::89] = 2**45 + 1
        v[3::101] = -(2**40)
        v[5::103] = 2**31 - 1
        v[7::107] = -(2**31)
        p = rng.integers(0, 10, n).astype(np.int32)
        _check_sga([(p, {"lo": 1})], [key], [v], C5_AGGS, expected_groups=G,
                   kernel="k_sga_bulk<Sig pred i32, key i64")


# ---------------------------------------------------------------- run-time compiled signatures (jit.cu)
JIT = "run-time compiled (NVRTC)"


@pytest.mark.parametrize("case", ["q1_one_key", "q1_minmax_other", "q1_f64_max", "two_values_tables",
                                  "i64_pred_tables", "no_pred_u8_key"])
def test_jit_signatures(case):
    """Plans no compiled-in signature matches get the same bulk kernel compiled by NVRTC for their
    signature (Ocelot's run-time kernel compilation): parity with the oracle and the
    kernel that ran."""
    n = 700_001
    li = _lineitem(n, datagen.BASE_SEED + 4, f64=True)
    vi = [li["quantity"], li["extendedprice"], li["discount"], li["tax"]]
    vf = [li["quantity_f"], li["extendedprice_f"], li["discount_f"], li["tax_f"]]
    pred = [(li["shipdate"], {"hi": 10471})]
    if case == "q1_one_key":             # GROUP BY l_returnflag only (3 groups)
        _check_sga(pred, [li["returnflag"]], vi, Q1_AGGS, expected_groups=4, order_by_key=True,
                   kernel=f"{JIT}; 4 private slots")
    elif case == "q1_minmax_other":      # Q1 + MIN(tax) + MAX(discount)
        _check_sga(pred, [li["returnflag"], li["linestatus"]], vi,
                   Q1_AGGS + [{"op": "min", "a": 3}, {"op": "max", "a": 2}], expected_groups=4,
                   order_by_key=True, kernel=f"{JIT}; 4 private slots")
    elif case == "q1_f64_max":           # fp64 Q1 + MAX(tax)
        _check_sga(pred, [li["returnflag"], li["linestatus"]], vf, Q1_AGGS_F64 + [{"op": "max", "a": 3}],
                   expected_groups=4, order_by_key=True, kernel=f"{JIT}; 4 private slots")
    elif case == "two_values_tables":    # C5-like with two value columns: CTA table
        sw = datagen.sweep_host(n, datagen.BASE_SEED + 5, 300, s=1.0)
        v2 = (sw["v"] * 3 - 7).astype(np.int64)
        aggs = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "max", "a": 1}, {"op": "min", "a": 1}]
        _check_sga([(sw["p"], {"hi": 799_999})], [sw["key"]], [sw["v"], v2], aggs, expected_groups=300,
                   kernel=f"{JIT}; CTA table")
    elif case == "i64_pred_tables":      # predicate on an int64 column, u8 x u8 keys, 12 groups
        rng = np.random.default_rng(4)
        k1, k2 = rng.integers(0, 4, n).astype(np.uint8), rng.integers(0, 3, n).astype(np.uint8)
        aggs = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "max", "a": 0}]
        _check_sga([(li["extendedprice"], {"lo": 1_000_000, "hi": 6_000_000})], [k1, k2], [li["quantity"]], aggs,
                   expected_groups=12, kernel=f"{JIT}; CTA table")
    else:                                # no predicate, one u8 key, fp64 values (private slots)
        aggs = [{"op": "sum", "a": 1}, {"op": "avg", "a": 0}, {"op": "count"}]
        _check_sga([], [li["linestatus"]], vf, aggs, expected_groups=2, kernel=f"{JIT}; 4 private slots")


def test_jit_off(monkeypatch):
    """OCL_NO_JIT: the same plan runs on the unified kernel (the fallback stays exact)."""
    monkeypatch.setenv("OCL_NO_JIT", "1")
    n = 100_003
    li = _lineitem(n, datagen.BASE_SEED + 4)
    vi = [li["quantity"], li["extendedprice"], li["discount"], li["tax"]]
    _check_sga([(li["shipdate"], {"hi": 10471})], [li["returnflag"]], vi, Q1_AGGS, expected_groups=4,
               kernel="k_sga<")


# ---------------------------------------------------------------- select-compact-gather (k_sga_sparse)
@pytest.mark.parametrize("G", [4, 16, 300, 2000])
@pytest.mark.parametrize("zipf,sel", [(0.0, 0.001), (1.0, 0.01), (1.5, 0.05), (0.0, 0.3)])
def test_c5_select_compact_gather(monkeypatch, G, zipf, sel):
    """k_sga_sparse: the ring carries the predicate column only; each warp compacts its qualifying rows from
    the ballot masks and gathers their key / value sectors (select -> prefix-sum
    compaction -> grouping, per stage).  OCL_SPARSE_PCT=100 forces it whenever the sample selects < 100 %."""
    monkeypatch.setenv("OCL_SPARSE_PCT", "100")
    n = (1 << 21) + 77                               # several batches per CTA and a ragged tail
    sw = datagen.sweep_host(n, datagen.BASE_SEED + 7, G, s=zipf)
    preds = [(sw["p"], {"hi": int(round(sel * 10**6)) - 1})]
    _check_sga(preds, [sw["key"]], [sw["v"]], C5_AGGS, expected_groups=G,
               kernel=f"k_sga_bulk<Sig pred i32, key i64, COUNT/SUM/MIN/MAX; {_c5_tier(G)}>")


@pytest.mark.parametrize("G", [4, 300])
def test_sparse_bitmap_and_exact_paths(monkeypatch, G):
    """Select-compact-gather with the bitmap output, values beyond int32 (exact per-row path), the key ~0
    and an empty selection."""
    monkeypatch.setenv("OCL_SPARSE_PCT", "100")
    n = 1_500_011
    rng = np.random.default_rng(G + 5)
    key = rng.integers(0, G, n).astype(np.int64) * 7919 - 3
    key[::1013] = -1
    v = rng.integers(-2**31, 2**31, n).astype(np.int64)
    v[::997] = 2**45 + 1
    p = rng.integers(0, 1000, n).astype(np.int32)
    for hi in (9, -1):                               # ~1 %, and nothing selected
        _check_sga([(p, {"hi": hi})], [key], [v], C5_AGGS, expected_groups=G, bitmap=True,
                   kernel="k_sga_bulk<Sig pred i32, key i64")


@pytest.mark.parametrize("f64", [False, True])
def test_q1_select_compact_gather(monkeypatch, f64):
    """The Q1 signatures (private tier) at ~2 % selectivity through the twin."""
    monkeypatch.setenv("OCL_SPARSE_PCT", "100")
    li = _lineitem(1_200_007, datagen.BASE_SEED + 8, f64=f64)
    p, k, v, a = _q1_plan(li, f64)
    p = [(li["shipdate"], {"hi": 8200})]
    _check_sga(p, k, v, a, order_by_key=True, kernel=f"k_sga_bulk<Sig Q1 {'fp64' if f64 else 'int64'}>")


def test_jit_select_compact_gather(monkeypatch):
    """A run-time compiled signature (two value columns, CTA table) through its compiled twin."""
    monkeypatch.setenv("OCL_SPARSE_PCT", "100")
    n = 900_001
    sw = datagen.sweep_host(n, datagen.BASE_SEED + 5, 300, s=1.0)
    v2 = (sw["v"] * 3 - 7).astype(np.int64)
    aggs = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "max", "a": 1}, {"op": "min", "a": 1}]
    _check_sga([(sw["p"], {"hi": 19_999})], [sw["key"]], [sw["v"], v2], aggs, expected_groups=300,
               kernel=f"{JIT}; CTA table")


def test_c5_sparse_default_threshold():
    """At 2^24 rows the default threshold (8 %) takes the twin for a 1 % predicate: full oracle compare."""
    n = (1 << 24) + 77
    sw = datagen.sweep_host(n, datagen.BASE_SEED + 9, 256, s=1.0)
    _check_sga([(sw["p"], {"hi": 9_999})], [sw["key"]], [sw["v"]], C5_AGGS, expected_groups=256,
               kernel="k_sga_bulk<Sig pred i32, key i64, COUNT/SUM/MIN/MAX; CTA table>")
