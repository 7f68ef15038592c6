"""Host-side checks without a GPU: the C-ABI library loads and exports every symbol
include/ocelot_b200.h declares; host-only entry points validate arguments."""
import ctypes
import os
import re

import numpy as np
import pytest
import torch

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


@pytest.fixture(scope="module")
def pkg():
    import subprocess
    lib = os.path.join(ROOT, "paper_journals_pvldb_heimelspmm13_b200", "_lib", "libocelot_b200.so")
    if not os.path.exists(lib):
        subprocess.run(["make", "-s", "-C", ROOT, "paper_journals_pvldb_heimelspmm13_b200/_lib/libocelot_b200.so"],
                       check=True)
    import paper_journals_pvldb_heimelspmm13_b200 as p
    return p


def declared_symbols():
    hdr = open(os.path.join(ROOT, "include", "ocelot_b200.h")).read()
    return sorted(set(re.findall(r"\b(ocl_[a-z0-9_]+)\s*\(", hdr)))


def test_header_symbols_exported(pkg):
    lib = pkg.lib()
    syms = declared_symbols()
    assert len(syms) >= 20
    for s in syms:
        assert hasattr(lib, s), s
    assert set(syms) == set(pkg.ABI_SYMBOLS)


def test_status_strings(pkg):
    lib = pkg.lib()
    assert lib.ocl_status_string(0) == b"OCL_OK"
    assert lib.ocl_status_string(3) == b"OCL_ERR_CAPACITY"
    assert lib.ocl_version() == 1


def _args(pkg, vals, aggs, keys=(), preds=()):
    keep = []
    vc = (pkg.Column * max(len(vals), 1))()
    for i, (ptr, dt, n) in enumerate(vals):
        vc[i] = pkg.Column(ptr, dt, 0, n)
    kc = (pkg.Column * max(len(keys), 1))()
    for i, (ptr, dt, n) in enumerate(keys):
        kc[i] = pkg.Column(ptr, dt, 0, n)
    ag = (pkg.Agg * max(len(aggs), 1))()
    for i, (op, expr, a, b, c, s) in enumerate(aggs):
        ag[i] = pkg.Agg(op, expr, a, b, c, s, 0x1000)
    a = pkg.SgaArgs()
    a.val_cols, a.nvals = ctypes.addressof(vc), len(vals)
    a.key_cols, a.nkeys = ctypes.addressof(kc), len(keys)
    a.aggs, a.naggs = ctypes.addressof(ag), len(aggs)
    a.expected_groups, a.out_capacity = 4, 16
    keep += [vc, kc, ag]
    return a, keep


def test_partial_row_bytes_layout(pkg):
    """Entry = key + count + per-value states (int SUM 16 B, f64 SUM 8 B, MIN/MAX 8 B), 32/64-aligned."""
    lib = pkg.lib()
    I64, F64 = 3, 4
    n = 100
    # Q1: 5 distinct int sums -> 16 + 5*16 = 96
    a, keep = _args(pkg, [(0x100, I64, n)] * 4,
                    [(1, 0, 0, -1, -1, 0), (1, 0, 1, -1, -1, 0), (1, 1, 1, 2, -1, 2), (1, 2, 1, 2, 3, 2),
                     (4, 0, 0, -1, -1, 0), (4, 0, 1, -1, -1, 0), (4, 0, 2, -1, -1, 0), (0, 0, -1, -1, -1, 0)])
    sz = ctypes.c_size_t()
    assert lib.ocl_partial_row_bytes(ctypes.byref(a), ctypes.byref(sz)) == 0
    assert sz.value == 96
    # count + sum + min + max of one int column: 16 + 16 + 8 + 8 = 48 -> 64
    a, keep = _args(pkg, [(0x100, I64, n)], [(0, 0, -1, -1, -1, 0), (1, 0, 0, -1, -1, 0), (2, 0, 0, -1, -1, 0),
                                             (3, 0, 0, -1, -1, 0)])
    assert lib.ocl_partial_row_bytes(ctypes.byref(a), ctypes.byref(sz)) == 0
    assert sz.value == 64
    # f64 sum only: 16 + 8 -> 32
    a, keep = _args(pkg, [(0x100, F64, n)], [(1, 0, 0, -1, -1, 0)])
    assert lib.ocl_partial_row_bytes(ctypes.byref(a), ctypes.byref(sz)) == 0
    assert sz.value == 32


@pytest.mark.parametrize("case,status", [
    ("mixed_expr", 1), ("u8_sum", 2), ("bad_index", 1), ("minmax_expr", 2), ("len_mismatch", 1),
    ("too_many_rows", 1), ("key_too_wide", 1), ("f64_key", 1), ("bad_scale", 1),
])
def test_argument_validation(pkg, case, status):
    lib = pkg.lib()
    U8, I32, I64, F64 = 1, 2, 3, 4
    n = 100
    vals = [(0x100, I64, n), (0x200, F64, n)]
    aggs = [(1, 0, 0, -1, -1, 0)]
    keys = []
    if case == "mixed_expr":
        aggs = [(1, 1, 0, 1, -1, 2)]
    elif case == "u8_sum":
        vals = [(0x100, U8, n)]
    elif case == "bad_index":
        aggs = [(1, 0, 7, -1, -1, 0)]
    elif case == "minmax_expr":
        vals = [(0x100, I64, n), (0x200, I64, n)]
        aggs = [(2, 1, 0, 1, -1, 2)]
    elif case == "len_mismatch":
        vals = [(0x100, I64, n), (0x200, I64, n + 1)]
    elif case == "too_many_rows":
        vals = [(0x100, I64, 1 << 32)]
    elif case == "key_too_wide":
        keys = [(0x300, I64, n), (0x400, U8, n)]
    elif case == "f64_key":
        keys = [(0x300, F64, n)]
    elif case == "bad_scale":
        vals = [(0x100, I64, n), (0x200, I64, n)]
        aggs = [(1, 1, 0, 1, -1, 19)]
    a, keep = _args(pkg, vals, aggs, keys)
    sz = ctypes.c_size_t()
    assert lib.ocl_partial_row_bytes(ctypes.byref(a), ctypes.byref(sz)) == status
    assert lib.ocl_last_error()


def test_no_cpu_fallback(pkg):
    """On a host without CUDA the product path must fail loudly, never compute on the CPU."""
    if torch.cuda.is_available():
        pytest.skip("GPU present")
    with pytest.raises(RuntimeError):
        pkg.select_bitmap(torch.zeros(10, dtype=torch.int32), {"hi": 3})


def test_product_does_not_import_oracle():
    """The CUDA path shares no code with the oracle (neither imports the other)."""
    pkgdir = os.path.join(ROOT, "paper_journals_pvldb_heimelspmm13_b200")
    for dirpath, _, files in os.walk(pkgdir):
        for f in files:
            if f.endswith((".py", ".cu", ".cuh", ".h", ".cpp")):
                src = open(os.path.join(dirpath, f)).read()
                assert not re.search(r"^\s*(import|from)\s+oracle", src, re.M), f
                assert "oracle.h" not in src, f
    osrc = open(os.path.join(ROOT, "oracle", "oracle.cpp")).read()
    assert "ocelot_b200.h" not in osrc and "common.cuh" not in osrc
