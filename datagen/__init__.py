"""Seeded synthetic inputs shared by the oracle side and the CUDA side.

This module holds none of the method's arithmetic: it only draws the
lineitem-shaped columns (SURVEY.md §8(d) recipe; TPC-H distributions cited by
the paper as [36]) and the cardinality-sweep columns from
the counter-based generator in ``ocl_datagen.h``.  The same C header is
compiled for the host (``liboclgen_host.so``) and for sm_100a
(``liboclgen_dev.so``), so a GPU rank generates its row shard in place and the
host regenerates identical rows for the oracle.

Config seeds: ``BASE_SEED + i`` for config Ci (i = 1..5).
"""
from __future__ import annotations

import ctypes
import os

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
BASE_SEED = 20130826
Q1_SHIP_CUTOFF = 10471          # date '1998-12-01' - 90 days, days since 1970-01-01
LINEITEM_INT_FIELDS = ("orderkey", "shipdate", "returnflag", "linestatus",
                       "quantity", "extendedprice", "discount", "tax")
LINEITEM_F64_FIELDS = ("quantity_f", "extendedprice_f", "discount_f", "tax_f")
_DTYPES = {"orderkey": np.int64, "shipdate": np.int32, "returnflag": np.uint8, "linestatus": np.uint8,
           "quantity": np.int64, "extendedprice": np.int64, "discount": np.int64, "tax": np.int64,
           "quantity_f": np.float64, "extendedprice_f": np.float64, "discount_f": np.float64,
           "tax_f": np.float64}
_ORDER = LINEITEM_INT_FIELDS + LINEITEM_F64_FIELDS

_host = None
_dev = None


def _load(name):
    path = os.path.join(_HERE, name)
    if not os.path.exists(path):
        raise RuntimeError(f"{path} missing: run `make` (or __graft_entry__.build()) first")
    return ctypes.CDLL(path)


def _host_lib():
    global _host
    if _host is None:
        _host = _load("liboclgen_host.so")
        u64 = ctypes.c_uint64
        _host.oclg_fill_lineitem.argtypes = [u64, u64, u64, u64, ctypes.c_int] + [ctypes.c_void_p] * 12
        _host.oclg_fill_lineitem.restype = None
        _host.oclg_zipf_cdf.argtypes = [u64, ctypes.c_double, ctypes.c_void_p]
        _host.oclg_fill_sweep.argtypes = [u64, u64, u64, u64, ctypes.c_void_p] + [ctypes.c_void_p] * 4
    return _host


def _dev_lib():
    global _dev
    if _dev is None:
        _dev = _load("liboclgen_dev.so")
        u64 = ctypes.c_uint64
        _dev.oclg_dev_fill_lineitem.argtypes = [u64, u64, u64, u64, ctypes.c_int] + [ctypes.c_void_p] * 13
        _dev.oclg_dev_fill_lineitem.restype = ctypes.c_int
        _dev.oclg_dev_fill_sweep.argtypes = [u64, u64, u64, u64, ctypes.c_void_p] + [ctypes.c_void_p] * 5
        _dev.oclg_dev_fill_sweep.restype = ctypes.c_int
    return _dev


def lineitem_host(n, seed, fields=LINEITEM_INT_FIELDS, row0=0, n_total=None, shuffled=False, out=None):
    """Rows [row0, row0+n) of the lineitem-shaped table as numpy arrays.

    ``n_total`` is the size of the whole table (sets the part count and the
    shuffle domain); it defaults to ``row0 + n``.  ``out`` may supply
    preallocated (e.g. pinned) arrays by field name.
    """
    n_total = row0 + n if n_total is None else n_total
    arrays = {}
    ptrs = []
    for f in _ORDER:
        if f in fields:
            a = out[f] if out is not None and f in out else np.empty(n, dtype=_DTYPES[f])
            assert a.dtype == _DTYPES[f] and a.shape[0] >= n and a.flags.c_contiguous
            arrays[f] = a
            ptrs.append(a.ctypes.data)
        else:
            ptrs.append(None)
    _host_lib().oclg_fill_lineitem(seed, row0, n, n_total, int(bool(shuffled)), *ptrs)
    return arrays


def lineitem_device(n, seed, fields=LINEITEM_INT_FIELDS, row0=0, n_total=None, shuffled=False, device=None):
    """Same rows as :func:`lineitem_host`, generated in place on the GPU (torch tensors)."""
    import torch
    n_total = row0 + n if n_total is None else n_total
    device = device or torch.device("cuda", torch.cuda.current_device())
    tdt = {np.int64: torch.int64, np.int32: torch.int32, np.uint8: torch.uint8, np.float64: torch.float64}
    tensors = {}
    ptrs = []
    for f in _ORDER:
        if f in fields:
            t = torch.empty(n, dtype=tdt[_DTYPES[f]], device=device)
            tensors[f] = t
            ptrs.append(t.data_ptr() if n else None)
        else:
            ptrs.append(None)
    stream = torch.cuda.current_stream(device).cuda_stream
    rc = _dev_lib().oclg_dev_fill_lineitem(seed, row0, n, n_total, int(bool(shuffled)), *ptrs, stream)
    if rc != 0:
        raise RuntimeError(f"device lineitem generation failed (cudaError {rc})")
    return tensors


def zipf_cdf(G, s):
    """Inverse-CDF table of Zipf(s) over G ranks (None for s == 0: uniform)."""
    if s == 0:
        return None
    cdf = np.empty(G, dtype=np.float64)
    _host_lib().oclg_zipf_cdf(G, float(s), cdf.ctypes.data)
    return cdf


def sweep_host(n, seed, G, s=0.0, row0=0, f64=False):
    """Cardinality-sweep columns (config C5): p i32, key i64, v i64 (+ v_f f64)."""
    cdf = zipf_cdf(G, s)
    p = np.empty(n, np.int32)
    key = np.empty(n, np.int64)
    v = np.empty(n, np.int64)
    v_f = np.empty(n, np.float64) if f64 else None
    _host_lib().oclg_fill_sweep(seed, row0, n, G, None if cdf is None else cdf.ctypes.data,
                                p.ctypes.data, key.ctypes.data, v.ctypes.data,
                                None if v_f is None else v_f.ctypes.data)
    out = {"p": p, "key": key, "v": v}
    if f64:
        out["v_f"] = v_f
    return out


def sweep_device(n, seed, G, s=0.0, row0=0, f64=False, device=None):
    import torch
    device = device or torch.device("cuda", torch.cuda.current_device())
    cdf = zipf_cdf(G, s)
    cdf_t = None if cdf is None else torch.from_numpy(cdf).to(device)
    p = torch.empty(n, dtype=torch.int32, device=device)
    key = torch.empty(n, dtype=torch.int64, device=device)
    v = torch.empty(n, dtype=torch.int64, device=device)
    v_f = torch.empty(n, dtype=torch.float64, device=device) if f64 else None
    stream = torch.cuda.current_stream(device).cuda_stream
    rc = _dev_lib().oclg_dev_fill_sweep(seed, row0, n, G, None if cdf_t is None else cdf_t.data_ptr(),
                                        p.data_ptr(), key.data_ptr(), v.data_ptr(),
                                        None if v_f is None else v_f.data_ptr(), stream)
    if rc != 0:
        raise RuntimeError(f"device sweep generation failed (cudaError {rc})")
    torch.cuda.current_stream(device).synchronize()
    out = {"p": p, "key": key, "v": v}
    if f64:
        out["v_f"] = v_f
    return out


def orders_keys(n_orders, seed=None, shuffled=True):
    """o_orderkey of the orders table behind a lineitem of 4 * n_orders rows: the sparse keys
    (o/8)*32 + o%8 + 1 of ocl_datagen.h (8 of every 32 used, dbgen-like), optionally in a seeded
    random row order.  int64 numpy array."""
    o = np.arange(n_orders, dtype=np.int64)
    k = (o // 8) * 32 + o % 8 + 1
    if shuffled:
        k = np.random.default_rng(BASE_SEED if seed is None else seed).permutation(k)
    return k
