"""Shared test helpers: golden loader, Q1 spec, per-key comparison rules."""
from __future__ import annotations

import os

import numpy as np

GOLDEN = os.path.join(os.path.dirname(os.path.abspath(__file__)), "golden")

Q1_CUTOFF = 10471
Q1_PRED = {"hi": Q1_CUTOFF, "hi_incl": True}
# vals = [quantity, extendedprice, discount, tax]
Q1_AGGS = [
    {"op": "sum", "expr": "col", "a": 0},                                          # sum_qty
    {"op": "sum", "expr": "col", "a": 1},                                          # sum_base_price
    {"op": "sum", "expr": "mul_1minus", "a": 1, "b": 2, "scale": 2},               # sum_disc_price
    {"op": "sum", "expr": "mul_1minus_1plus", "a": 1, "b": 2, "c": 3, "scale": 2},  # sum_charge
    {"op": "avg", "expr": "col", "a": 0},                                          # avg_qty
    {"op": "avg", "expr": "col", "a": 1},                                          # avg_price
    {"op": "avg", "expr": "col", "a": 2},                                          # avg_disc
    {"op": "count"},                                                               # count_order
]
Q1_AGGS_F64 = [dict(a, scale=0) if a.get("expr", "col") != "col" else dict(a) for a in Q1_AGGS]


def load_golden(name="q1_worked_example.txt"):
    sec = None
    out = {"rows": [], "intermediates": {}, "groups": []}
    with open(os.path.join(GOLDEN, name)) as f:
        for line in f:
            line = line.strip()
            if not line or line.startswith("#"):
                continue
            if line.startswith("["):
                sec = line.strip("[]")
                continue
            parts = line.split()
            if sec == "rows":
                out["rows"].append(parts)
            elif sec == "intermediates":
                out["intermediates"][parts[0]] = parts[1:]
            elif sec == "groups":
                out["groups"].append(parts)
    return out


def golden_columns(g):
    rows = g["rows"]
    cols = {
        "shipdate": np.array([int(r[1]) for r in rows], np.int32),
        "returnflag": np.array([ord(r[2]) for r in rows], np.uint8),
        "linestatus": np.array([ord(r[3]) for r in rows], np.uint8),
        "quantity": np.array([int(r[4]) for r in rows], np.int64),
        "extendedprice": np.array([int(r[5]) for r in rows], np.int64),
        "discount": np.array([int(r[6]) for r in rows], np.int64),
        "tax": np.array([int(r[7]) for r in rows], np.int64),
    }
    return cols


def int128_list(words):
    w = np.asarray(words, dtype=np.uint64).reshape(-1, 2)
    out = []
    for lo, hi in w:
        v = (int(hi) << 64) | int(lo)
        if v >= 1 << 127:
            v -= 1 << 128
        out.append(v)
    return out


def by_key(keys, outs, aggs, vals_dtypes):
    """Map packed key -> tuple of per-aggregate Python values (int128 decoded)."""
    res = {}
    dec = []
    for spec, o in zip(aggs, outs):
        fp = spec["op"] != "count" and vals_dtypes[spec["a"]] == np.float64
        if spec["op"] == "sum" and not fp:
            dec.append(int128_list(o))
        else:
            dec.append([x.item() for x in np.asarray(o)])
    for i, k in enumerate(np.asarray(keys)):
        res[int(np.uint64(k))] = tuple(d[i] for d in dec)
    return res


def assert_results_equal(got, ref, aggs, vals_dtypes, rtol=1e-9):
    """Rules of SURVEY §8(c): ints/COUNT/MIN/MAX bit-exact; fp64 SUM/AVG within rtol
    relative per group (AVG of ints: expected exact, enforced <= rtol)."""
    assert set(got) == set(ref), f"group key sets differ: extra {set(got) - set(ref)}, missing {set(ref) - set(got)}"
    for k in ref:
        for i, spec in enumerate(aggs):
            g, r = got[k][i], ref[k][i]
            fp_in = spec["op"] != "count" and vals_dtypes[spec["a"]] == np.float64
            if spec["op"] == "avg" or (spec["op"] == "sum" and fp_in):
                assert abs(g - r) <= rtol * abs(r) + 1e-300, f"key {k:#x} agg {i} {spec}: {g!r} vs {r!r}"
            else:
                assert g == r, f"key {k:#x} agg {i} {spec}: {g!r} vs {r!r}"


def canon_gids(gids):
    """Relabel a gid column by first occurrence (SURVEY §8(c) comparison rule for gids)."""
    gids = np.asarray(gids)
    mapping = {}
    out = np.empty(len(gids), np.int64)
    for j, g in enumerate(gids.tolist()):
        if g not in mapping:
            mapping[g] = len(mapping)
        out[j] = mapping[g]
    return out


def assert_results_equal_np(gkeys, gouts, rkeys, routs, aggs, vals_dtypes, rtol=1e-9):
    """Vectorised version of assert_results_equal for large G: sort both sides by key."""
    gk = np.asarray(gkeys).view(np.uint64)
    rk = np.asarray(rkeys).view(np.uint64)
    assert len(gk) == len(rk), f"G differs: {len(gk)} vs {len(rk)}"
    gi, ri = np.argsort(gk, kind="stable"), np.argsort(rk, kind="stable")
    assert np.array_equal(gk[gi], rk[ri]), "group key sets differ"
    for spec, g, r in zip(aggs, gouts, routs):
        g, r = np.asarray(g)[gi], np.asarray(r)[ri]
        fp_in = spec["op"] != "count" and vals_dtypes[spec["a"]] == np.float64
        if spec["op"] == "avg" or (spec["op"] == "sum" and fp_in):
            assert np.all(np.abs(g - r) <= rtol * np.abs(r)), spec
        else:
            assert np.array_equal(g.view(np.uint64) if g.dtype != np.uint64 else g,
                                  r.view(np.uint64) if r.dtype != np.uint64 else r), spec
