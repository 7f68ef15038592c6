"""CPU oracle — TEST INFRASTRUCTURE ONLY.

ctypes wrapper over ``liboracle.so`` (``oracle.cpp``): a plain, slow,
single-threaded C++17 implementation of Ocelot's select -> hash GROUP BY ->
aggregate path (Heimel et al., PVLDB 6(9) 2013; §4.1) with the
readings of SURVEY.md §8(c).  It shares no code with the CUDA product path.

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py``'s
``cpu_baseline`` / ``--impl reference`` legs may import this package.

Spec conventions (plain dicts, parsed independently by each side):
  range: {"lo": x|None, "hi": x|None, "lo_incl": bool, "hi_incl": bool, "anti": bool}
  agg:   {"op": "count"|"sum"|"min"|"max"|"avg", "expr": "col"|"mul_1minus"|"mul_1minus_1plus",
          "a": i, "b": j, "c": k, "scale": s}
Outputs: COUNT int64[G]; SUM of int -> int128 as uint64[G, 2] (lo, hi words, see
``int128``); SUM of f64 -> float64[G]; MIN/MAX -> int64 or float64; AVG -> float64.
"""
from __future__ import annotations

import ctypes
import os

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_lib = None

ORC_DTYPE = {np.dtype(np.uint8): 1, np.dtype(np.int32): 2, np.dtype(np.int64): 3, np.dtype(np.float64): 4}
OPS = {"count": 0, "sum": 1, "min": 2, "max": 3, "avg": 4}
EXPRS = {"col": 0, "mul_1minus": 1, "mul_1minus_1plus": 2}


class _Col(ctypes.Structure):
    _fields_ = [("data", ctypes.c_void_p), ("dtype", ctypes.c_int32), ("pad_", ctypes.c_int32),
                ("n", ctypes.c_int64)]


class _Range(ctypes.Structure):
    _fields_ = [("dtype", ctypes.c_int32), ("has_lo", ctypes.c_uint8), ("has_hi", ctypes.c_uint8),
                ("lo_incl", ctypes.c_uint8), ("hi_incl", ctypes.c_uint8), ("anti", ctypes.c_uint8),
                ("pad_", ctypes.c_uint8 * 7), ("lo_i", ctypes.c_int64), ("hi_i", ctypes.c_int64),
                ("lo_f", ctypes.c_double), ("hi_f", ctypes.c_double)]


class _Agg(ctypes.Structure):
    _fields_ = [("op", ctypes.c_int32), ("expr", ctypes.c_int32), ("a", ctypes.c_int32), ("b", ctypes.c_int32),
                ("c", ctypes.c_int32), ("decimal_scale", ctypes.c_int32), ("out", ctypes.c_void_p)]


def lib():
    global _lib
    if _lib is None:
        path = os.path.join(_HERE, "liboracle.so")
        if not os.path.exists(path):
            raise RuntimeError(f"{path} missing: run `make` (or __graft_entry__.build()) first")
        L = ctypes.CDLL(path)
        P = ctypes.c_void_p
        L.oracle_select.argtypes = [P, P, P]
        L.oracle_select.restype = ctypes.c_int
        L.oracle_bitmap_combine.argtypes = [ctypes.c_int, P, P, P, ctypes.c_int64]
        L.oracle_compact.argtypes = [P, ctypes.c_int64, P]
        L.oracle_compact.restype = ctypes.c_int64
        L.oracle_gather.argtypes = [P, P, ctypes.c_int64, P]
        for f in (L.oracle_group_hash, L.oracle_group_sort, L.oracle_group_sorted):
            f.argtypes = [P, ctypes.c_int, P, ctypes.c_int64, P, P]
            f.restype = ctypes.c_int64
        L.oracle_hash_join.argtypes = [P, P, P, ctypes.c_int64, P, P, ctypes.c_int64]
        L.oracle_hash_join.restype = ctypes.c_int64
        L.oracle_aggregate.argtypes = [P, P, ctypes.c_int64, ctypes.c_int64, P, ctypes.c_int, P, ctypes.c_int]
        L.oracle_aggregate.restype = ctypes.c_int
        L.oracle_sga.argtypes = [P, P, ctypes.c_int, P, ctypes.c_int, P, ctypes.c_int, P, ctypes.c_int,
                                 ctypes.c_int, P, ctypes.c_int64]
        L.oracle_sga.restype = ctypes.c_int64
        _lib = L
    return _lib


def _col(a):
    a = np.ascontiguousarray(a)
    return _Col(a.ctypes.data, ORC_DTYPE[a.dtype], 0, a.shape[0]), a


def _range(spec, dtype):
    r = _Range()
    r.dtype = ORC_DTYPE[np.dtype(dtype)]
    lo, hi = spec.get("lo"), spec.get("hi")
    r.has_lo, r.has_hi = int(lo is not None), int(hi is not None)
    r.lo_incl, r.hi_incl = int(spec.get("lo_incl", True)), int(spec.get("hi_incl", True))
    r.anti = int(spec.get("anti", False))
    if np.dtype(dtype) == np.float64:
        r.lo_f = float(lo) if lo is not None else 0.0
        r.hi_f = float(hi) if hi is not None else 0.0
    else:
        r.lo_i = int(lo) if lo is not None else 0
        r.hi_i = int(hi) if hi is not None else 0
    return r


def _out_array(spec, vals, G):
    op = spec["op"]
    if op == "count":
        return np.zeros(max(G, 1), np.int64)
    a = vals[spec["a"]]
    fp = a.dtype == np.float64
    if op == "sum":
        return np.zeros(max(G, 1), np.float64) if fp else np.zeros((max(G, 1), 2), np.uint64)
    if op == "avg":
        return np.zeros(max(G, 1), np.float64)
    return np.zeros(max(G, 1), np.float64 if fp else np.int64)


def _aggs(specs, vals, G):
    arr = (_Agg * max(len(specs), 1))()
    outs = []
    for i, s in enumerate(specs):
        o = _out_array(s, vals, G)
        outs.append(o)
        arr[i] = _Agg(OPS[s["op"]], EXPRS[s.get("expr", "col")], s.get("a", -1), s.get("b", -1), s.get("c", -1),
                      s.get("scale", 0), o.ctypes.data)
    return arr, outs


def int128(words):
    """uint64[G, 2] (lo, hi two's complement) -> list of Python ints."""
    w = np.asarray(words, dtype=np.uint64).reshape(-1, 2)
    out = []
    for lo, hi in w:
        v = (int(hi) << 64) | int(lo)
        if v >= 1 << 127:
            v -= 1 << 128
        out.append(v)
    return out


def select(col, pred):
    c, keep = _col(col)
    words = (c.n + 31) // 32
    bm = np.zeros(max(words, 1), np.uint32)
    r = _range(pred, keep.dtype)
    if lib().oracle_select(ctypes.byref(c), ctypes.byref(r), bm.ctypes.data) != 0:
        raise ValueError("invalid select spec")
    return bm[:words]


def bitmap_combine(op, a, b, n):
    words = (n + 31) // 32
    out = np.zeros(max(words, 1), np.uint32)
    opi = {"and": 0, "or": 1, "andnot": 2}[op]
    a = np.ascontiguousarray(a, np.uint32)
    b = np.ascontiguousarray(b, np.uint32)
    lib().oracle_bitmap_combine(opi, a.ctypes.data, b.ctypes.data, out.ctypes.data, n)
    return out[:words]


def compact(bitmap, n):
    bm = np.ascontiguousarray(bitmap, np.uint32)
    oids = np.zeros(max(n, 1), np.uint32)
    m = lib().oracle_compact(bm.ctypes.data, n, oids.ctypes.data)
    return oids[:m].copy()


def gather(col, oids):
    c, keep = _col(col)
    oids = np.ascontiguousarray(oids, np.uint32)
    out = np.zeros(max(len(oids), 1), keep.dtype)
    lib().oracle_gather(ctypes.byref(c), oids.ctypes.data, len(oids), out.ctypes.data)
    return out[:len(oids)]


def _group(fn, keys, oids, m):
    cols = (_Col * len(keys))()
    keep = []
    for i, k in enumerate(keys):
        cols[i], a = _col(k)
        keep.append(a)
    if oids is not None:
        oids = np.ascontiguousarray(oids, np.uint32)
        m = len(oids)
    gids = np.zeros(max(m, 1), np.int32)
    keys_out = np.zeros(max(m, 1), np.int64)
    G = fn(cols, len(keys), None if oids is None else oids.ctypes.data, m, gids.ctypes.data, keys_out.ctypes.data)
    if G == -2:
        raise ValueError("keys not sorted (non-decreasing packed key required)")
    if G < 0:
        raise ValueError("invalid group spec")
    return gids[:m].copy(), keys_out[:G].copy()


def group_hash(keys, oids=None, m=None):
    """First-occurrence dense gids (MonetDB group.group) via std::unordered_map."""
    return _group(lib().oracle_group_hash, keys, oids, len(keys[0]) if m is None else m)


def group_sort(keys, oids=None, m=None):
    """Independent sort-based grouping; must equal group_hash exactly."""
    return _group(lib().oracle_group_sort, keys, oids, len(keys[0]) if m is None else m)


def group_sorted(keys, oids=None, m=None):
    """The paper's sorted-input grouping (successor compare + prefix sum, L554-556); raises on unsorted keys."""
    return _group(lib().oracle_group_sorted, keys, oids, len(keys[0]) if m is None else m)


def hash_join(build, probe, oids=None):
    """All (probe row, build row) pairs with equal keys, probe order, partners ascending -> two uint32 arrays."""
    b, kb = _col(build)
    p, kp = _col(probe)
    m = len(probe)
    if oids is not None:
        oids = np.ascontiguousarray(oids, np.uint32)
        m = len(oids)
    n = lib().oracle_hash_join(ctypes.byref(b), ctypes.byref(p), None if oids is None else oids.ctypes.data, m,
                               None, None, 0)
    if n < 0:
        raise ValueError("invalid join spec")
    op, ob = np.zeros(max(n, 1), np.uint32), np.zeros(max(n, 1), np.uint32)
    lib().oracle_hash_join(ctypes.byref(b), ctypes.byref(p), None if oids is None else oids.ctypes.data, m,
                           op.ctypes.data, ob.ctypes.data, n)
    return op[:n], ob[:n]


def aggregate(gids, G, vals, aggs, oids=None):
    cols = (_Col * max(len(vals), 1))()
    keep = []
    for i, v in enumerate(vals):
        cols[i], a = _col(v)
        keep.append(a)
    gids = np.ascontiguousarray(gids, np.int32)
    m = len(gids)
    if oids is not None:
        oids = np.ascontiguousarray(oids, np.uint32)
    arr, outs = _aggs(aggs, keep, G)
    rc = lib().oracle_aggregate(gids.ctypes.data, None if oids is None else oids.ctypes.data, m, G, cols,
                                len(vals), arr, len(aggs))
    if rc != 0:
        raise ValueError("invalid aggregate spec")
    return [o[:G] for o in outs]


def sga(preds, keys, vals, aggs, order_by_key=False):
    """Fused reference: preds = [(column, range_spec)], keys = [column], vals = [column].
    Returns (keys_out int64[G], [outputs])."""
    n = None
    for c in [p[0] for p in preds] + list(keys) + list(vals):
        n = len(c)
    n = 0 if n is None else n
    pcols = (_Col * max(len(preds), 1))()
    pr = (_Range * max(len(preds), 1))()
    keep = []
    for i, (c, spec) in enumerate(preds):
        pcols[i], a = _col(c)
        keep.append(a)
        pr[i] = _range(spec, a.dtype)
    kcols = (_Col * max(len(keys), 1))()
    for i, c in enumerate(keys):
        kcols[i], a = _col(c)
        keep.append(a)
    vcols = (_Col * max(len(vals), 1))()
    vkeep = []
    for i, c in enumerate(vals):
        vcols[i], a = _col(c)
        vkeep.append(a)
    cap = max(n, 1)
    arr, outs = _aggs(aggs, vkeep, cap)
    keys_out = np.zeros(cap, np.int64)
    G = lib().oracle_sga(pcols, pr, len(preds), kcols, len(keys), vcols, len(vals), arr, len(aggs),
                         int(bool(order_by_key)), keys_out.ctypes.data, cap)
    if G < 0:
        raise ValueError(f"invalid sga spec ({G})")
    return keys_out[:G].copy(), [o[:G].copy() for o in outs]
