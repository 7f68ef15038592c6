"""Pins of the CPU oracle against things other than itself (no GPU needed).

Each test pins one oracle function to what the paper and the mathematics fix:
the hand-computed worked example (tests/golden), brute force on tiny inputs in
pure Python, closed forms, library routines for special cases, invariants.
"""
from fractions import Fraction

import numpy as np
import pytest

import oracle
from tests._common import (Q1_AGGS, Q1_PRED, assert_results_equal, by_key, golden_columns, int128_list,
                           load_golden)

DT = [np.uint8, np.int32, np.int64, np.float64]


# ---------------------------------------------------------------- worked example
def test_worked_example_intermediates():
    g = load_golden()
    c = golden_columns(g)
    n = len(c["shipdate"])
    bm = oracle.select(c["shipdate"], Q1_PRED)
    assert int(bm[0]) == int(g["intermediates"]["bitmap_word0"][0], 16)
    oids = oracle.compact(bm, n)
    assert oids.tolist() == [int(x) for x in g["intermediates"]["oids"]]
    gids, keys = oracle.group_hash([c["returnflag"], c["linestatus"]], oids)
    assert gids.tolist() == [int(x) for x in g["intermediates"]["gids_first_occurrence"]]
    assert [hex(k) for k in keys] == ["0x4e4f", "0x5246", "0x4146", "0x4e46"]


def test_worked_example_q1_outputs():
    g = load_golden()
    c = golden_columns(g)
    vals = [c["quantity"], c["extendedprice"], c["discount"], c["tax"]]
    aggs = Q1_AGGS + [{"op": "sum", "a": 2}, {"op": "min", "a": 0}, {"op": "max", "a": 0}]
    keys, outs = oracle.sga([(c["shipdate"], Q1_PRED)], [c["returnflag"], c["linestatus"]], vals, aggs,
                            order_by_key=True)
    assert keys.tolist() == [0x4146, 0x4E46, 0x4E4F, 0x5246]            # ORDER BY rf, ls
    got = by_key(keys, outs, aggs, [v.dtype for v in vals])
    # golden columns: key count sum_qty sum_price sum_dp sum_charge sum_disc min max avg_qty avg_price avg_disc
    ref = {}
    for row in g["groups"]:
        k = int(row[0], 16)
        cnt, sq, sp, sdp, sch, sd, mn, mx = (int(x) for x in row[1:9])
        aq, ap, ad = (float(x) for x in row[9:12])
        ref[k] = (sq, sp, sdp, sch, aq, ap, ad, cnt, sd, mn, mx)
    assert_results_equal(got, ref, aggs, [v.dtype for v in vals], rtol=0.0)
    # key (A,O) = 0x414F occurs only in a filtered-out row (s18)
    assert 0x414F not in got


def test_worked_example_f64_variant():
    """fp64 columns = decimals / 100: charge sums within 1e-15 of the exact decimal (s10, §8(c))."""
    g = load_golden()
    c = golden_columns(g)
    vals = [c[k].astype(np.float64) / 100.0 for k in ("quantity", "extendedprice", "discount", "tax")]
    aggs = [{"op": "sum", "expr": "mul_1minus_1plus", "a": 1, "b": 2, "c": 3, "scale": 0}]
    keys, outs = oracle.sga([(c["shipdate"], Q1_PRED)], [c["returnflag"], c["linestatus"]], vals, aggs,
                            order_by_key=True)
    exact = {0x4146: Fraction(70047433344, 10**6), 0x4E46: Fraction(21363713280, 10**6),
             0x4E4F: Fraction(111664744920, 10**6), 0x5246: Fraction(59287896576, 10**6)}
    for k, v in zip(keys.tolist(), outs[0].tolist()):
        assert abs(Fraction(v) - exact[k]) <= Fraction(1, 10**15) * exact[k]


def test_worked_example_f64_all_branches():
    """Every fp64 branch of the oracle's aggregation on the worked example (fp64 columns = decimals / 100,
    S = 1.0): SUM of a column, SUM of a*(S-b) (MUL_1MINUS) and a*(S-b)*(S+c) (MUL_1MINUS_1PLUS), AVG = SUM /
    COUNT.  Pinned to the hand-computed exact decimals of tests/golden (not to a re-typed formula): each
    fp64 row value is within a few ulps of its exact decimal and every value is >= 0, so each output lies
    within 1e-14 (relative) of the exact rational.  A dropped term, a sign error, a wrong operand index or
    an AVG divided by the wrong count misses by far more than that."""
    g = load_golden()
    c = golden_columns(g)
    names = ("quantity", "extendedprice", "discount", "tax")
    vals = [c[k].astype(np.float64) / 100.0 for k in names]
    aggs = [{"op": "sum", "a": 0}, {"op": "sum", "a": 1},
            {"op": "sum", "expr": "mul_1minus", "a": 1, "b": 2, "scale": 0},
            {"op": "sum", "expr": "mul_1minus_1plus", "a": 1, "b": 2, "c": 3, "scale": 0},
            {"op": "avg", "a": 0}, {"op": "avg", "a": 1}, {"op": "avg", "a": 2},
            {"op": "avg", "expr": "mul_1minus", "a": 1, "b": 2, "scale": 0}, {"op": "count"}]
    keys, outs = oracle.sga([(c["shipdate"], Q1_PRED)], [c["returnflag"], c["linestatus"]], vals, aggs,
                            order_by_key=True)
    for i, k in enumerate(keys.tolist()):
        row = next(r for r in g["groups"] if int(r[0], 16) == k)
        cnt, sq, sp, sdp, sch, sd = (int(x) for x in row[1:7])
        exact = [Fraction(sq, 100), Fraction(sp, 100), Fraction(sdp, 10**4), Fraction(sch, 10**6),
                 Fraction(sq, 100 * cnt), Fraction(sp, 100 * cnt), Fraction(sd, 100 * cnt),
                 Fraction(sdp, 10**4 * cnt)]
        for j, e in enumerate(exact):
            v = outs[j][i].item()
            assert abs(Fraction(v) - e) <= Fraction(1, 10**14) * e, (hex(k), aggs[j], v, float(e))
        assert outs[8][i] == cnt


@pytest.mark.parametrize("scale", [0, 2])
def test_f64_expressions_exact_decimal(scale):
    """fp64 MUL_1MINUS / MUL_1MINUS_1PLUS sums and AVG on random decimals k/100 against exact rationals
    (Python Fractions from the integers k), S = 10^scale, one and several groups."""
    rng = np.random.default_rng(scale + 11)
    n = 2000
    ka, kb, kc = rng.integers(1, 10**6, n), rng.integers(0, 11, n), rng.integers(0, 9, n)
    vals = [ka.astype(np.float64) / 100.0, kb.astype(np.float64) / 100.0, kc.astype(np.float64) / 100.0]
    gk = (ka % 3).astype(np.int64)
    aggs = [{"op": "sum", "expr": "mul_1minus", "a": 0, "b": 1, "scale": scale},
            {"op": "sum", "expr": "mul_1minus_1plus", "a": 0, "b": 1, "c": 2, "scale": scale},
            {"op": "avg", "expr": "mul_1minus", "a": 0, "b": 1, "scale": scale}, {"op": "avg", "a": 2}]
    keys, outs = oracle.sga([], [gk], vals, aggs)
    S = 10**scale
    for i, k in enumerate(keys.tolist()):
        sel = gk == k
        a = [Fraction(int(x), 100) for x in ka[sel]]
        b = [Fraction(int(x), 100) for x in kb[sel]]
        cc = [Fraction(int(x), 100) for x in kc[sel]]
        m1 = sum(x * (S - y) for x, y in zip(a, b))
        m2 = sum(x * (S - y) * (S + z) for x, y, z in zip(a, b, cc))
        exact = [m1, m2, m1 / len(a), sum(cc) / len(a)]
        for j, e in enumerate(exact):
            v = outs[j][i].item()
            assert abs(Fraction(v) - e) <= Fraction(1, 10**13) * abs(e), (k, aggs[j], v, float(e))


# ---------------------------------------------------------------- selection
def _py_pred(x, spec):
    ok = True
    if spec.get("lo") is not None:
        ok = ok and (x >= spec["lo"] if spec.get("lo_incl", True) else x > spec["lo"])
    if spec.get("hi") is not None:
        ok = ok and (x <= spec["hi"] if spec.get("hi_incl", True) else x < spec["hi"])
    return (not ok) if spec.get("anti", False) else ok


@pytest.mark.parametrize("dtype", DT)
def test_select_brute_force(dtype):
    rng = np.random.default_rng(7)
    n = 333
    if dtype == np.float64:
        col = rng.integers(-50, 50, n).astype(np.float64) / 4.0
        bounds = [-3.25, 0.0, 2.5]
    elif dtype == np.uint8:
        col = rng.integers(0, 256, n).astype(np.uint8)
        bounds = [0, 17, 200, 255]
    else:
        col = rng.integers(-60, 60, n).astype(dtype)
        bounds = [-5, 0, 7]
    for lo in [None] + bounds:
        for hi in [None] + bounds:
            for lo_incl in (True, False):
                for hi_incl in (True, False):
                    for anti in (False, True):
                        spec = {"lo": lo, "hi": hi, "lo_incl": lo_incl, "hi_incl": hi_incl, "anti": anti}
                        bm = oracle.select(col, spec)
                        bits = [(int(bm[r >> 5]) >> (r & 31)) & 1 for r in range(n)]
                        assert bits == [int(_py_pred(x, spec)) for x in col.tolist()], spec
                        assert int(bm[-1]) >> (n & 31) == 0          # tail bits zero


def test_select_special_cases():
    col = np.arange(100, dtype=np.int32)
    n = 100
    allones = oracle.select(col, {})
    assert allones.tolist() == [0xFFFFFFFF] * 3 + [0xF]                 # unbounded: all ones, zero tail
    assert oracle.select(col, {"lo": 50, "hi": 10}).tolist() == [0] * 4  # lo > hi: empty
    a = oracle.select(col, {"lo": 10, "hi": 70})
    b = oracle.select(col, {"lo": 10, "hi": 70, "anti": True})
    assert ((a ^ b) == allones).all()                                   # anti = complement within n
    pt = oracle.select(col, {"lo": 42, "hi": 42})                        # point select
    assert oracle.compact(pt, n).tolist() == [42]


@pytest.mark.parametrize("n", [0, 1, 99, 100, 101, 150, 12345])
def test_select_popcount_closed_form(n):
    p = (np.arange(n) % 100).astype(np.int32)
    bm = oracle.select(p, {"hi": 49})
    pop = sum(bin(int(w)).count("1") for w in bm)
    assert pop == 50 * (n // 100) + min(n % 100, 50)


def test_bitmap_combine():
    rng = np.random.default_rng(3)
    n = 200
    x = rng.integers(0, 10, n).astype(np.int32)
    a = oracle.select(x, {"hi": 5})
    b = oracle.select(x, {"lo": 3})
    assert (oracle.bitmap_combine("and", a, b, n) == oracle.select(x, {"lo": 3, "hi": 5})).all()
    assert (oracle.bitmap_combine("or", a, b, n) == oracle.select(x, {})).all()
    assert (oracle.bitmap_combine("andnot", a, b, n) == oracle.select(x, {"hi": 2})).all()


# ---------------------------------------------------------------- compaction
@pytest.mark.parametrize("n", [0, 1, 31, 32, 33, 1000, 4097])
def test_compact_matches_numpy(n):
    rng = np.random.default_rng(n)
    bits = rng.random(n) < 0.37
    words = np.zeros((n + 31) // 32, np.uint32)
    for r in np.flatnonzero(bits):
        words[r >> 5] |= np.uint32(1 << (r & 31))
    oids = oracle.compact(words, n)
    assert oids.tolist() == np.flatnonzero(bits).tolist()               # library routine
    assert len(oids) == sum(bin(int(w)).count("1") for w in words)      # m = popcount
    assert all(np.diff(oids.astype(np.int64)) > 0)                      # strictly ascending


def test_gather():
    col = np.arange(50, dtype=np.int64) * 3 + 1
    oids = np.array([0, 7, 7, 49], np.uint32)
    assert oracle.gather(col, oids).tolist() == [1, 22, 22, 148]


# ---------------------------------------------------------------- grouping
def _nested_loop_group(keys):
    """O(n*G) brute force: first-occurrence gids."""
    seen = []
    gids = []
    for k in keys:
        for g, s in enumerate(seen):
            if s == k:
                gids.append(g)
                break
        else:
            seen.append(k)
            gids.append(len(seen) - 1)
    return gids, seen


@pytest.mark.parametrize("kind", ["u8", "i32", "i64", "u8u8", "i32i32", "u8i32", "i64neg"])
def test_group_brute_force_and_sort(kind):
    rng = np.random.default_rng(11)
    n = 1500
    if kind == "u8":
        keys = [rng.integers(0, 256, n).astype(np.uint8)]
        packed = [int(x) for x in keys[0]]
    elif kind == "i32":
        keys = [rng.integers(-20, 20, n).astype(np.int32)]
        packed = [int(x) & 0xFFFFFFFF for x in keys[0]]
    elif kind == "i64":
        keys = [rng.integers(0, 40, n).astype(np.int64) * 10**15]
        packed = [int(x) for x in keys[0]]
    elif kind == "i64neg":
        keys = [rng.integers(-30, 30, n).astype(np.int64)]
        packed = [int(x) & 0xFFFFFFFFFFFFFFFF for x in keys[0]]
    elif kind == "u8u8":
        keys = [rng.choice(np.array([65, 78, 82], np.uint8), n), rng.choice(np.array([70, 79], np.uint8), n)]
        packed = [(int(a) << 8) | int(b) for a, b in zip(*keys)]
    elif kind == "i32i32":
        keys = [rng.integers(-3, 3, n).astype(np.int32), rng.integers(-3, 3, n).astype(np.int32)]
        packed = [((int(a) & 0xFFFFFFFF) << 32) | (int(b) & 0xFFFFFFFF) for a, b in zip(*keys)]
    else:
        keys = [rng.integers(0, 4, n).astype(np.uint8), rng.integers(-2, 2, n).astype(np.int32)]
        packed = [(int(a) << 32) | (int(b) & 0xFFFFFFFF) for a, b in zip(*keys)]
    oids = np.flatnonzero(rng.random(n) < 0.8).astype(np.uint32)
    sel = [packed[int(o)] for o in oids]
    ref_gids, ref_keys = _nested_loop_group(sel)
    gh, kh = oracle.group_hash(keys, oids)
    gs, ks = oracle.group_sort(keys, oids)
    assert gh.tolist() == ref_gids and gs.tolist() == ref_gids
    assert [int(np.uint64(k)) for k in kh] == ref_keys
    assert [int(np.uint64(k)) for k in ks] == ref_keys
    assert len(kh) == len(set(sel))                                     # G = |distinct qualifying keys|


def test_group_invalid_key_width():
    a = np.zeros(4, np.int64)
    with pytest.raises(ValueError):
        oracle.group_hash([a, a])                                       # 128 packed bits > 64


def test_group_degenerate():
    x = np.arange(100, dtype=np.int64)
    g, k = oracle.group_hash([x])
    assert g.tolist() == list(range(100)) and k.tolist() == list(range(100))   # all distinct: G = m
    g, k = oracle.group_hash([np.full(100, 5, np.int32)])
    assert g.tolist() == [0] * 100 and k.tolist() == [5]                        # single key: G = 1


# ---------------------------------------------------------------- aggregation
@pytest.mark.parametrize("n,G", [(1, 1), (10, 3), (1000, 7), (4096, 64), (777, 1000)])
def test_aggregate_closed_form(n, G):
    """keys r mod G, values r, all rows: c_g = floor((n-1-g)/G)+1, SUM_g = c_g*g + G*c_g(c_g-1)/2,
    MIN_g = g, MAX_g = g + (c_g-1)G (SURVEY §8(c) pins)."""
    r = np.arange(n, dtype=np.int64)
    keys = (r % G).astype(np.int64)
    gids, kout = oracle.group_hash([keys])
    aggs = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "min", "a": 0}, {"op": "max", "a": 0},
            {"op": "avg", "a": 0}]
    outs = oracle.aggregate(gids, len(kout), [r], aggs)
    for gi, k in enumerate(kout.tolist()):
        c = (n - 1 - k) // G + 1
        assert outs[0][gi] == c
        assert int128_list(outs[1])[gi] == c * k + G * c * (c - 1) // 2
        assert outs[2][gi] == k
        assert outs[3][gi] == k + (c - 1) * G
        assert outs[4][gi] == float(Fraction(c * k + G * c * (c - 1) // 2, c))


def test_aggregate_ungrouped_reduces_to_library():
    rng = np.random.default_rng(5)
    v = rng.integers(-10**12, 10**12, 5000).astype(np.int64)
    f = rng.standard_normal(5000)
    gids = np.zeros(5000, np.int32)
    outs = oracle.aggregate(gids, 1, [v, f], [{"op": "sum", "a": 0}, {"op": "min", "a": 0}, {"op": "max", "a": 0},
                                              {"op": "min", "a": 1}, {"op": "max", "a": 1}, {"op": "sum", "a": 1}])
    assert int128_list(outs[0])[0] == sum(int(x) for x in v)
    assert outs[1][0] == v.min() and outs[2][0] == v.max()
    assert outs[3][0] == f.min() and outs[4][0] == f.max()
    exact = sum(Fraction(float(x)) for x in f)
    assert abs(Fraction(float(outs[5][0])) - exact) <= Fraction(1, 10**12) * sum(abs(Fraction(float(x))) for x in f)


def test_int128_sum_beyond_int64():
    """s11: int64 SUM accumulates in int128 (Q1 sum_charge at SF100 exceeds INT64_MAX)."""
    v = np.full(1000, 2**62 + 12345, np.int64)
    v[::3] = -(2**63)
    gids = np.zeros(1000, np.int32)
    s = int128_list(oracle.aggregate(gids, 1, [v], [{"op": "sum", "a": 0}])[0])[0]
    assert s == sum(int(x) for x in v)
    avg = oracle.aggregate(gids, 1, [v], [{"op": "avg", "a": 0}])[0][0]
    assert avg == float(s) / 1000.0     # Python int->float is correctly rounded: pins int128->double


def test_int_expressions_wrap_mod_2_128():
    rng = np.random.default_rng(9)
    a = rng.integers(-2**62, 2**62, 300).astype(np.int64)
    b = rng.integers(-2**62, 2**62, 300).astype(np.int64)
    c = rng.integers(-2**62, 2**62, 300).astype(np.int64)
    gids = np.zeros(300, np.int32)
    aggs = [{"op": "sum", "expr": "mul_1minus", "a": 0, "b": 1, "scale": 3},
            {"op": "sum", "expr": "mul_1minus_1plus", "a": 0, "b": 1, "c": 2, "scale": 2}]
    outs = oracle.aggregate(gids, 1, [a, b, c], aggs)

    def wrap(x):
        x %= 1 << 128
        return x - (1 << 128) if x >= 1 << 127 else x
    e1 = wrap(sum(int(x) * (1000 - int(y)) for x, y in zip(a, b)))
    e2 = wrap(sum(int(x) * (100 - int(y)) * (100 + int(z)) for x, y, z in zip(a, b, c)))
    assert int128_list(outs[0])[0] == e1
    assert int128_list(outs[1])[0] == e2


def test_f64_sum_pinned_by_exact_integer_sum():
    """Values k/100 from integers k: the fp64 SUM is within ~1e-15 of the exact decimal sum."""
    rng = np.random.default_rng(2)
    k = rng.integers(0, 10**7, 20000).astype(np.int64)
    gids = (np.arange(20000) % 4).astype(np.int32)
    outs = oracle.aggregate(gids, 4, [k.astype(np.float64) / 100.0], [{"op": "sum", "a": 0}])
    for g in range(4):
        exact = Fraction(int(k[g::4].sum()), 100)
        assert abs(Fraction(float(outs[0][g])) - exact) <= Fraction(1, 10**15) * exact


def test_sga_invariants_on_generated_lineitem():
    import datagen
    n = 20000
    li = datagen.lineitem_host(n, datagen.BASE_SEED + 1)
    vals = [li["quantity"], li["extendedprice"], li["discount"], li["tax"]]
    keys, outs = oracle.sga([(li["shipdate"], Q1_PRED)], [li["returnflag"], li["linestatus"]], vals, Q1_AGGS)
    bm = oracle.select(li["shipdate"], Q1_PRED)
    pop = sum(bin(int(w)).count("1") for w in bm)
    assert int(outs[7].sum()) == pop                                     # sum of COUNTs = popcount
    sel = li["shipdate"] <= 10471
    distinct = set(((li["returnflag"][sel].astype(np.int64) << 8) | li["linestatus"][sel]).tolist())
    assert set(keys.tolist()) == distinct                               # group set = distinct qualifying keys
    # brute-force Python sums per key
    for gi, k in enumerate(keys.tolist()):
        m = sel & (((li["returnflag"].astype(np.int64) << 8) | li["linestatus"]) == k)
        assert int128_list(outs[0])[gi] == int(li["quantity"][m].sum())
        p, d, t = (li[f][m].astype(object) for f in ("extendedprice", "discount", "tax"))
        assert int128_list(outs[3])[gi] == int(sum(p * (100 - d) * (100 + t)))


def test_sga_empty_selection_and_order():
    x = np.arange(64, dtype=np.int32)
    keys, outs = oracle.sga([(x, {"lo": 100})], [x], [x.astype(np.int64)], [{"op": "count"}])
    assert len(keys) == 0 and len(outs[0]) == 0                         # s17: G = 0
    k = np.array([5, 3, 9, 3, 5, 0xFF], np.uint8)
    keys, outs = oracle.sga([], [k], [k.astype(np.int64)], [{"op": "count"}], order_by_key=True)
    assert keys.tolist() == [3, 5, 9, 255] and outs[0].tolist() == [2, 2, 1, 1]


def test_sga_ungrouped():
    v = np.arange(10, dtype=np.int64)
    keys, outs = oracle.sga([(v, {"lo": 3})], [], [v], [{"op": "sum", "a": 0}, {"op": "count"}])
    assert keys.tolist() == [0] and int128_list(outs[0]) == [42] and outs[1].tolist() == [7]


# ---------------------------------------------------------------- sorted-input grouping
def _py_distinct_prefix(keys):
    """Brute force for sorted keys: gid[j] = (number of distinct keys among rows 0..j) - 1."""
    seen, out = set(), []
    for k in keys:
        seen.add(int(k))
        out.append(len(seen) - 1)
    return out


@pytest.mark.parametrize("n", [0, 1, 2, 7, 64, 257, 3000])
def test_group_sorted_brute_force_and_hash(n):
    rng = np.random.default_rng(1000 + n)
    keys = np.sort(rng.integers(0, max(n // 3, 1), n)).astype(np.int64)
    gids, kout = oracle.group_sorted([keys])
    assert gids.tolist() == _py_distinct_prefix(keys)
    assert kout.tolist() == sorted(set(keys.tolist()))                  # ascending, one per group
    hg, hk = oracle.group_hash([keys])                                   # first occurrence == run order
    assert gids.tolist() == hg.tolist() and kout.tolist() == hk.tolist()


def test_group_sorted_two_columns_and_oids():
    rng = np.random.default_rng(7)
    a = np.sort(rng.integers(0, 5, 500)).astype(np.uint8)               # sorted (a, b) pairs
    b = np.concatenate([np.sort(rng.integers(0, 4, int((a == v).sum()))) for v in range(5)]).astype(np.uint8)
    oids = np.flatnonzero(rng.random(500) < 0.3).astype(np.uint32)       # a subsequence stays sorted
    gids, kout = oracle.group_sorted([a, b], oids)
    packed = [(int(a[o]) << 8) | int(b[o]) for o in oids]
    assert gids.tolist() == _py_distinct_prefix(packed)
    assert kout.tolist() == sorted(set(packed))


def test_group_sorted_degenerate_and_unsorted():
    one = np.full(100, 42, np.int64)
    gids, kout = oracle.group_sorted([one])
    assert gids.tolist() == [0] * 100 and kout.tolist() == [42]
    distinct = np.arange(50, dtype=np.int32)
    gids, kout = oracle.group_sorted([distinct])
    assert gids.tolist() == list(range(50)) and kout.tolist() == list(range(50))
    with pytest.raises(ValueError, match="not sorted"):
        oracle.group_sorted([np.array([1, 2, 1], np.int64)])
    # unsigned packed order: -1 (all ones) sorts after every non-negative key
    gids, kout = oracle.group_sorted([np.array([0, 5, -1, -1], np.int64)])
    assert gids.tolist() == [0, 1, 2, 2]


# ---------------------------------------------------------------- equi hash join
def _py_nested_join(build, probe):
    """Brute-force nested loop (the paper's theta-join shape with '=')."""
    return [(j, i) for j in range(len(probe)) for i in range(len(build)) if build[i] == probe[j]]


@pytest.mark.parametrize("dtype", [np.uint8, np.int32, np.int64])
def test_hash_join_nested_loop(dtype):
    rng = np.random.default_rng(3)
    build = rng.integers(0, 40, 150).astype(dtype)
    probe = rng.integers(0, 60, 200).astype(dtype)
    op, ob = oracle.hash_join(build, probe)
    assert list(zip(op.tolist(), ob.tolist())) == _py_nested_join(build.tolist(), probe.tolist())


def test_hash_join_pk_fk_and_oids():
    rng = np.random.default_rng(4)
    pk = rng.permutation(1000).astype(np.int64) * 7 - 3000               # unique build keys, some negative
    fk = rng.choice(pk, 5000)
    fk[::10] = 10**9                                                      # dangling foreign keys
    oids = np.flatnonzero(rng.random(5000) < 0.5).astype(np.uint32)
    op, ob = oracle.hash_join(pk, fk, oids)
    pos = {int(k): i for i, k in enumerate(pk.tolist())}
    ref = [(int(j), pos[int(fk[j])]) for j in oids.tolist() if int(fk[j]) in pos]
    assert list(zip(op.tolist(), ob.tolist())) == ref                    # <= 1 partner per probe row (PK)
    assert len(ref) == sum(1 for j in oids.tolist() if fk[j] != 10**9)
    with pytest.raises(ValueError):
        oracle.hash_join(pk, fk.astype(np.int32))                         # dtypes differ
