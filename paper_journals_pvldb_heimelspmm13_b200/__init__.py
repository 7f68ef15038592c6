"""ocelot-b200: B200-native select -> hash GROUP BY -> aggregate (Ocelot, Heimel et al., PVLDB 2013).

Thin Python binding over the C ABI of ``_lib/libocelot_b200.so``
(``include/ocelot_b200.h``): argument marshalling only — every step of the path
runs in the library's sm_100a CUDA kernels.  PyTorch supplies device memory,
streams and ``torch.distributed`` (plumbing).  There is no CPU fallback: if the
library or a CUDA device is missing, every call raises.

Function names follow the ABI (``ocl_select_bitmap`` -> :func:`select_bitmap` ...).
Spec conventions (plain dicts):
  range: {"lo": x|None, "hi": x|None, "lo_incl": bool, "hi_incl": bool, "anti": bool}
  agg:   {"op": "count"|"sum"|"min"|"max"|"avg", "expr": "col"|"mul_1minus"|"mul_1minus_1plus",
          "a": i, "b": j, "c": k, "scale": s}
Outputs: COUNT int64[G]; SUM of ints int64[G, 2] (int128 lo/hi words); SUM of f64
float64[G]; MIN/MAX int64 or float64; AVG float64.
"""
from __future__ import annotations

import ctypes
import os

import torch

_HERE = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.environ.get("OCL_LIB_PATH") or os.path.join(_HERE, "_lib", "libocelot_b200.so")

(OCL_OK, OCL_ERR_INVALID_ARG, OCL_ERR_UNSUPPORTED, OCL_ERR_CAPACITY, OCL_ERR_OUT_OF_MEMORY, OCL_ERR_CUDA,
 OCL_ERR_NCCL) = range(7)
_DTYPE = {torch.uint8: 1, torch.int32: 2, torch.int64: 3, torch.float64: 4}
_OPS = {"count": 0, "sum": 1, "min": 2, "max": 3, "avg": 4}
_EXPRS = {"col": 0, "mul_1minus": 1, "mul_1minus_1plus": 2}
_COMBINE = {"and": 0, "or": 1, "andnot": 2}


class OcelotError(RuntimeError):
    def __init__(self, status, msg):
        super().__init__(f"{_STATUS_NAMES.get(status, status)}: {msg}")
        self.status = status


_STATUS_NAMES = {0: "OCL_OK", 1: "OCL_ERR_INVALID_ARG", 2: "OCL_ERR_UNSUPPORTED", 3: "OCL_ERR_CAPACITY",
                 4: "OCL_ERR_OUT_OF_MEMORY", 5: "OCL_ERR_CUDA", 6: "OCL_ERR_NCCL"}


class Column(ctypes.Structure):
    _fields_ = [("data", ctypes.c_void_p), ("dtype", ctypes.c_int32), ("reserved", ctypes.c_int32),
                ("n", ctypes.c_int64)]


class Range(ctypes.Structure):
    _fields_ = [("dtype", ctypes.c_int32), ("has_lo", ctypes.c_uint8), ("has_hi", ctypes.c_uint8),
                ("lo_incl", ctypes.c_uint8), ("hi_incl", ctypes.c_uint8), ("anti", ctypes.c_uint8),
                ("reserved", ctypes.c_uint8 * 7), ("lo_i", ctypes.c_int64), ("hi_i", ctypes.c_int64),
                ("lo_f", ctypes.c_double), ("hi_f", ctypes.c_double)]


class Agg(ctypes.Structure):
    _fields_ = [("op", ctypes.c_int32), ("expr", ctypes.c_int32), ("a", ctypes.c_int32), ("b", ctypes.c_int32),
                ("c", ctypes.c_int32), ("decimal_scale", ctypes.c_int32), ("out", ctypes.c_void_p)]


class SgaArgs(ctypes.Structure):
    _fields_ = [("pred_cols", ctypes.c_void_p), ("preds", ctypes.c_void_p), ("npreds", ctypes.c_int32),
                ("nkeys", ctypes.c_int32), ("key_cols", ctypes.c_void_p), ("val_cols", ctypes.c_void_p),
                ("nvals", ctypes.c_int32), ("naggs", ctypes.c_int32), ("aggs", ctypes.c_void_p),
                ("expected_groups", ctypes.c_int64), ("out_capacity", ctypes.c_int64),
                ("keys_out", ctypes.c_void_p), ("ngroups_out", ctypes.c_void_p), ("bitmap_out", ctypes.c_void_p),
                ("dev_status", ctypes.c_void_p), ("order_by_key", ctypes.c_int32), ("tier", ctypes.c_int32),
                ("key_sorted", ctypes.c_int32), ("distributed", ctypes.c_int32)]


_lib = None


def lib():
    """Load the CUDA library (fails loudly: there is no CPU path)."""
    global _lib
    if _lib is None:
        if not os.path.exists(LIB_PATH):
            raise RuntimeError(f"{LIB_PATH} not built: run `make` or __graft_entry__.build()")
        L = ctypes.CDLL(LIB_PATH)
        P, I32, I64, SZ = ctypes.c_void_p, ctypes.c_int32, ctypes.c_int64, ctypes.c_size_t
        PSZ = ctypes.POINTER(ctypes.c_size_t)
        sig = {
            "ocl_ctx_create": [ctypes.c_int, ctypes.POINTER(ctypes.c_void_p)],
            "ocl_ctx_destroy": [P],
            "ocl_select_bitmap": [P, P, P, P, P],
            "ocl_bitmap_combine": [P, I32, P, P, P, I64, P],
            "ocl_prefix_compact_workspace_size": [P, I64, PSZ],
            "ocl_prefix_compact": [P, P, I64, P, P, P, SZ, P],
            "ocl_gather": [P, P, P, P, I64, P, P],
            "ocl_group_build_workspace_size": [P, I64, I64, PSZ],
            "ocl_group_build": [P, P, I32, P, P, I64, I64, P, P, I64, P, P, P, SZ, P],
            "ocl_group_build_paper_workspace_size": [P, I64, I64, PSZ],
            "ocl_group_build_paper": [P, P, I32, P, P, I64, I64, P, P, I64, P, P, P, SZ, P],
            "ocl_group_build_sorted_workspace_size": [P, I64, PSZ],
            "ocl_group_build_sorted": [P, P, I32, P, P, I64, P, P, I64, P, P, P, SZ, P],
            "ocl_group_aggregate_workspace_size": [P, I64, P, I32, P, I32, PSZ],
            "ocl_group_aggregate": [P, P, P, P, I64, P, I64, P, I32, P, I32, P, SZ, P],
            "ocl_select_group_aggregate_workspace_size": [P, P, PSZ],
            "ocl_select_group_aggregate": [P, P, P, SZ, P],
            "ocl_select_group_aggregate_sync_workspace_size": [P, P, PSZ],
            "ocl_select_group_aggregate_sync": [P, P, P, SZ, P],
            "ocl_ctx_set_phase_events": [P, I32, P, P],
            "ocl_nccl_unique_id": [P],
            "ocl_ctx_attach_nccl": [P, P, I32, I32],
            "ocl_ctx_nccl_rank": [P, ctypes.POINTER(I32), ctypes.POINTER(I32)],
            "ocl_partial_row_bytes": [P, PSZ],
            "ocl_sga_partial": [P, P, P, I64, P, P, SZ, P],
            "ocl_merge_partials_workspace_size": [P, P, I32, I64, PSZ],
            "ocl_merge_partials": [P, P, P, I32, I64, P, P, SZ, P],
            "ocl_radix_sort_workspace_size": [P, I64, I32, I32, PSZ],
            "ocl_radix_sort": [P, P, I32, P, P, P, P, P, SZ, P],
            "ocl_join_build_workspace_size": [P, I64, PSZ],
            "ocl_join_build": [P, P, P, SZ, P, P],
            "ocl_join_probe_workspace_size": [P, I64, PSZ],
            "ocl_join_probe": [P, P, P, P, P, P, I64, I32, P, P, I64, P, P, P, SZ, P],
            "ocl_route_partials_workspace_size": [P, I32, PSZ],
            "ocl_route_partials": [P, P, P, I64, I32, I32, P, P, P, SZ, P],
            "ocl_select_group_aggregate_host_workspace_size": [P, P, I64, PSZ],
            "ocl_select_group_aggregate_host": [P, P, I64, P, SZ, P],
        }
        for name, args in sig.items():
            if not hasattr(L, name):     # an older library build (A/B timing through OCL_LIB_PATH)
                continue
            f = getattr(L, name)
            f.argtypes = args
            f.restype = ctypes.c_int
        L.ocl_status_string.restype = ctypes.c_char_p
        L.ocl_last_error.restype = ctypes.c_char_p
        L.ocl_version.restype = ctypes.c_int32
        L.ocl_launch_count.restype = ctypes.c_uint64
        L.ocl_ctx_last_kernel.argtypes = [P]
        L.ocl_ctx_last_kernel.restype = ctypes.c_char_p
        L.ocl_ctx_set_kernel_events.argtypes = [P, P, P]
        L.ocl_ctx_set_kernel_events.restype = ctypes.c_int
        _lib = L
    return _lib


ABI_SYMBOLS = ("ocl_ctx_create", "ocl_ctx_destroy", "ocl_status_string", "ocl_last_error", "ocl_version",
               "ocl_launch_count", "ocl_ctx_last_kernel", "ocl_ctx_set_kernel_events",
               "ocl_select_bitmap", "ocl_bitmap_combine", "ocl_prefix_compact_workspace_size", "ocl_prefix_compact",
               "ocl_gather", "ocl_group_build_workspace_size", "ocl_group_build",
               "ocl_group_build_sorted_workspace_size", "ocl_group_build_sorted",
               "ocl_group_build_paper_workspace_size", "ocl_group_build_paper",
               "ocl_group_aggregate_workspace_size", "ocl_group_aggregate",
               "ocl_select_group_aggregate_workspace_size", "ocl_select_group_aggregate",
               "ocl_select_group_aggregate_sync_workspace_size", "ocl_select_group_aggregate_sync",
               "ocl_ctx_set_phase_events", "ocl_nccl_unique_id", "ocl_ctx_attach_nccl", "ocl_ctx_nccl_rank",
               "ocl_partial_row_bytes",
               "ocl_sga_partial", "ocl_merge_partials_workspace_size", "ocl_merge_partials",
               "ocl_route_partials_workspace_size", "ocl_route_partials",
               "ocl_join_build_workspace_size", "ocl_join_build", "ocl_join_probe_workspace_size", "ocl_join_probe",
               "ocl_radix_sort_workspace_size", "ocl_radix_sort",
               "ocl_select_group_aggregate_host_workspace_size", "ocl_select_group_aggregate_host")


def _check(status):
    if status != OCL_OK:
        raise OcelotError(status, lib().ocl_last_error().decode())


class Context:
    """Owns an ``ocl_ctx`` (device properties, grid sizing, internal copy streams)."""

    def __init__(self, device=None):
        if not torch.cuda.is_available():
            raise RuntimeError("ocelot-b200 needs a CUDA device (B200, sm_100a); there is no CPU fallback")
        self.device = torch.device("cuda", torch.cuda.current_device() if device is None else device)
        h = ctypes.c_void_p()
        _check(lib().ocl_ctx_create(self.device.index, ctypes.byref(h)))
        self.handle = h

    def __del__(self):
        if getattr(self, "handle", None) and _lib is not None:
            _lib.ocl_ctx_destroy(self.handle)
            self.handle = None

    def attach_nccl(self, unique_id, rank, nranks):
        """ocl_ctx_attach_nccl: join an NCCL communicator (collective over the nranks ranks)."""
        buf = ctypes.create_string_buffer(bytes(unique_id), 128)
        _check(lib().ocl_ctx_attach_nccl(self.handle, buf, int(rank), int(nranks)))

    @property
    def nccl_rank(self):
        r, n = ctypes.c_int32(), ctypes.c_int32()
        _check(lib().ocl_ctx_nccl_rank(self.handle, ctypes.byref(r), ctypes.byref(n)))
        return r.value, n.value


def nccl_unique_id():
    """ocl_nccl_unique_id: 128 bytes to hand to every rank (out of band)."""
    buf = ctypes.create_string_buffer(128)
    _check(lib().ocl_nccl_unique_id(buf))
    return buf.raw


_ctxs = {}


def launch_count():
    """Kernels launched by the library so far (process-wide)."""
    return int(lib().ocl_launch_count())


def last_kernel(ctx):
    """Name of the fused kernel instantiation the last fused call on ctx used."""
    return lib().ocl_ctx_last_kernel(ctx.handle).decode()


def set_phase_events(ctx, phase, begin=None, end=None):
    """Bracket phase 0 (fused kernel) or 1 (exchange + merge) of subsequent calls on ctx with events."""
    _check(lib().ocl_ctx_set_phase_events(ctx.handle, int(phase), begin.cuda_event if begin is not None else None,
                                          end.cuda_event if end is not None else None))


def set_kernel_events(ctx, begin=None, end=None):
    """Bracket the fused kernel of subsequent calls on ctx with torch.cuda.Event objects (or None)."""
    _check(lib().ocl_ctx_set_kernel_events(ctx.handle, begin.cuda_event if begin is not None else None,
                                           end.cuda_event if end is not None else None))


def context(device=None):
    idx = torch.cuda.current_device() if device is None else torch.device(device).index
    if idx not in _ctxs:
        _ctxs[idx] = Context(idx)
    return _ctxs[idx]


def _stream(stream):
    return (stream or torch.cuda.current_stream()).cuda_stream


def _col(t):
    if t.dtype not in _DTYPE:
        raise TypeError(f"unsupported column dtype {t.dtype}")
    if t.dim() != 1 or not t.is_contiguous():
        raise ValueError("columns must be 1-D contiguous tensors")
    return Column(t.data_ptr() if t.numel() else None, _DTYPE[t.dtype], 0, t.numel())


def _cols(ts):
    arr = (Column * max(len(ts), 1))()
    for i, t in enumerate(ts):
        arr[i] = _col(t)
    return arr


def _range(spec, dtype):
    r = Range()
    r.dtype = _DTYPE[dtype]
    lo, hi = spec.get("lo"), spec.get("hi")
    r.has_lo, r.has_hi = int(lo is not None), int(hi is not None)
    r.lo_incl, r.hi_incl = int(spec.get("lo_incl", True)), int(spec.get("hi_incl", True))
    r.anti = int(spec.get("anti", False))
    if dtype == torch.float64:
        r.lo_f = float(lo) if lo is not None else 0.0
        r.hi_f = float(hi) if hi is not None else 0.0
    else:
        r.lo_i = int(lo) if lo is not None else 0
        r.hi_i = int(hi) if hi is not None else 0
    return r


def _agg_out(spec, vals, cap, device):
    op = spec["op"]
    cap = max(cap, 1)
    if op == "count":
        return torch.zeros(cap, dtype=torch.int64, device=device)
    fp = vals[spec["a"]].dtype == torch.float64
    if op == "sum":
        return torch.zeros(cap, dtype=torch.float64, device=device) if fp else \
            torch.zeros((cap, 2), dtype=torch.int64, device=device)
    if op == "avg":
        return torch.zeros(cap, dtype=torch.float64, device=device)
    return torch.zeros(cap, dtype=torch.float64 if fp else torch.int64, device=device)


def _aggs(specs, vals, cap, device, outs=None):
    arr = (Agg * max(len(specs), 1))()
    outs = outs if outs is not None else [_agg_out(s, vals, cap, device) for s in specs]
    for i, s in enumerate(specs):
        arr[i] = Agg(_OPS[s["op"]], _EXPRS[s.get("expr", "col")], s.get("a", -1), s.get("b", -1), s.get("c", -1),
                     s.get("scale", 0), outs[i].data_ptr())
    return arr, outs


def _workspace(nbytes, device):
    return torch.empty(max(int(nbytes), 256), dtype=torch.uint8, device=device)


# ---------------------------------------------------------------- a1 / A2
def select_bitmap(col, pred, out=None, stream=None):
    """Predicate -> LSB-first uint32 bitmap (returned as int32 words)."""
    ctx = context(col.device)
    words = (col.numel() + 31) // 32
    out = out if out is not None else torch.empty(max(words, 1), dtype=torch.int32, device=col.device)
    c = _col(col)
    r = _range(pred, col.dtype)
    _check(lib().ocl_select_bitmap(ctx.handle, ctypes.byref(c), ctypes.byref(r), out.data_ptr(), _stream(stream)))
    return out[:words]


def bitmap_combine(op, a, b, n, out=None, stream=None):
    ctx = context(a.device)
    words = (n + 31) // 32
    out = out if out is not None else torch.empty(max(words, 1), dtype=torch.int32, device=a.device)
    _check(lib().ocl_bitmap_combine(ctx.handle, _COMBINE[op], a.data_ptr(), b.data_ptr(), out.data_ptr(), n,
                                    _stream(stream)))
    return out[:words]


# ---------------------------------------------------------------- a2 / a3
def prefix_compact(bitmap, n, stream=None):
    """Bitmap -> ascending oids (int32 storage of uint32) and device count m (int64[1])."""
    ctx = context(bitmap.device)
    sz = ctypes.c_size_t()
    _check(lib().ocl_prefix_compact_workspace_size(ctx.handle, n, ctypes.byref(sz)))
    ws = _workspace(sz.value, bitmap.device)
    oids = torch.empty(max(n, 1), dtype=torch.int32, device=bitmap.device)
    m = torch.zeros(1, dtype=torch.int64, device=bitmap.device)
    _check(lib().ocl_prefix_compact(ctx.handle, bitmap.data_ptr(), n, oids.data_ptr(), m.data_ptr(), ws.data_ptr(),
                                    sz.value, _stream(stream)))
    return oids, m


def gather(col, oids, m=None, max_m=None, stream=None):
    ctx = context(col.device)
    max_m = oids.numel() if max_m is None else max_m
    out = torch.empty(max(max_m, 1), dtype=col.dtype, device=col.device)
    c = _col(col)
    _check(lib().ocl_gather(ctx.handle, ctypes.byref(c), oids.data_ptr(), None if m is None else m.data_ptr(), max_m,
                            out.data_ptr(), _stream(stream)))
    return out


# ---------------------------------------------------------------- a4-a6
def group_build(keys, oids=None, m=None, max_rows=None, expected_groups=1024, out_capacity=None, stream=None,
                scheme="b200"):
    """Hash group-by -> (gids int32[max_rows], keys_out int64[cap], ngroups int64[1], status int32[1]).
    scheme "paper": the paper's optimistic / verify / pessimistic hashing, for the ablation."""
    dev = keys[0].device
    ctx = context(dev)
    max_rows = (oids.numel() if oids is not None else keys[0].numel()) if max_rows is None else max_rows
    out_capacity = max_rows if out_capacity is None else out_capacity
    sz = ctypes.c_size_t()
    ws_fn = lib().ocl_group_build_paper_workspace_size if scheme == "paper" else lib().ocl_group_build_workspace_size
    build_fn = lib().ocl_group_build_paper if scheme == "paper" else lib().ocl_group_build
    _check(ws_fn(ctx.handle, max_rows, expected_groups, ctypes.byref(sz)))
    ws = _workspace(sz.value, dev)
    gids = torch.empty(max(max_rows, 1), dtype=torch.int32, device=dev)
    keys_out = torch.empty(max(out_capacity, 1), dtype=torch.int64, device=dev)
    ng = torch.zeros(1, dtype=torch.int64, device=dev)
    status = torch.zeros(1, dtype=torch.int32, device=dev)
    kc = _cols(keys)
    _check(build_fn(ctx.handle, kc, len(keys), None if oids is None else oids.data_ptr(),
                                 None if m is None else m.data_ptr(), max_rows, expected_groups, gids.data_ptr(),
                                 keys_out.data_ptr(), out_capacity, ng.data_ptr(), status.data_ptr(), ws.data_ptr(),
                                 sz.value, _stream(stream)))
    return gids, keys_out, ng, status


def group_build_sorted(keys, oids=None, m=None, max_rows=None, out_capacity=None, stream=None):
    """Sorted-input group-by (successor compare + prefix sum) -> (gids int32[max_rows],
    keys_out int64[cap], ngroups int64[1], status int32[1]); gids ascend with the key."""
    dev = keys[0].device
    ctx = context(dev)
    max_rows = (oids.numel() if oids is not None else keys[0].numel()) if max_rows is None else max_rows
    out_capacity = max_rows if out_capacity is None else out_capacity
    sz = ctypes.c_size_t()
    _check(lib().ocl_group_build_sorted_workspace_size(ctx.handle, max_rows, ctypes.byref(sz)))
    ws = _workspace(sz.value, dev)
    gids = torch.empty(max(max_rows, 1), dtype=torch.int32, device=dev)
    keys_out = torch.empty(max(out_capacity, 1), dtype=torch.int64, device=dev)
    ng = torch.zeros(1, dtype=torch.int64, device=dev)
    status = torch.zeros(1, dtype=torch.int32, device=dev)
    kc = _cols(keys)
    _check(lib().ocl_group_build_sorted(ctx.handle, kc, len(keys), None if oids is None else oids.data_ptr(),
                                        None if m is None else m.data_ptr(), max_rows, gids.data_ptr(),
                                        keys_out.data_ptr(), out_capacity, ng.data_ptr(), status.data_ptr(),
                                        ws.data_ptr(), sz.value, _stream(stream)))
    return gids, keys_out, ng, status


# ---------------------------------------------------------------- radix sort
def radix_sort(keys, payload=None, rowids=False, stream=None):
    """Stable sort by the packed key (1-2 integer columns, unsigned order) -> (packed keys int64[n],
    payload permuted or None, source row ids int32[n] (uint32) or None)."""
    dev = keys[0].device
    ctx = context(dev)
    n = keys[0].numel()
    sz = ctypes.c_size_t()
    _check(lib().ocl_radix_sort_workspace_size(ctx.handle, n, int(payload is not None), int(bool(rowids)),
                                               ctypes.byref(sz)))
    ws = _workspace(sz.value, dev)
    ko = torch.empty(max(n, 1), dtype=torch.int64, device=dev)
    po = torch.empty(max(n, 1), dtype=payload.dtype, device=dev) if payload is not None else None
    ro = torch.empty(max(n, 1), dtype=torch.int32, device=dev) if rowids else None
    kc = _cols(keys)
    pc = _col(payload) if payload is not None else None
    _check(lib().ocl_radix_sort(ctx.handle, kc, len(keys), ctypes.byref(pc) if pc is not None else None,
                                ko.data_ptr(), po.data_ptr() if po is not None else None,
                                ro.data_ptr() if ro is not None else None, ws.data_ptr(), sz.value, _stream(stream)))
    return ko[:n], (po[:n] if po is not None else None), (ro[:n] if ro is not None else None)


# ---------------------------------------------------------------- equi hash join
class JoinBuild:
    """Hash table over a build key column (kept on the device for any number of probes)."""

    def __init__(self, build_key, stream=None):
        self.key = build_key
        self.ctx = context(build_key.device)
        self._kc = _col(build_key)
        sz = ctypes.c_size_t()
        _check(lib().ocl_join_build_workspace_size(self.ctx.handle, build_key.numel(), ctypes.byref(sz)))
        self.ws = _workspace(sz.value, build_key.device)
        self.status = torch.zeros(1, dtype=torch.int32, device=build_key.device)
        _check(lib().ocl_join_build(self.ctx.handle, ctypes.byref(self._kc), self.ws.data_ptr(), sz.value,
                                    self.status.data_ptr(), _stream(stream)))

    def probe(self, probe_key, oids=None, m=None, max_rows=None, pk_build=False, out_capacity=None, stream=None):
        """-> (out_probe int32[cap] (uint32 oids), out_build int32[cap], npairs int64[1], status int32[1])."""
        dev = probe_key.device
        max_rows = (oids.numel() if oids is not None else probe_key.numel()) if max_rows is None else max_rows
        out_capacity = max(max_rows, 1) if out_capacity is None else out_capacity
        sz = ctypes.c_size_t()
        _check(lib().ocl_join_probe_workspace_size(self.ctx.handle, max_rows, ctypes.byref(sz)))
        ws = _workspace(sz.value, dev)
        op = torch.empty(max(out_capacity, 1), dtype=torch.int32, device=dev)
        ob = torch.empty(max(out_capacity, 1), dtype=torch.int32, device=dev)
        nout = torch.zeros(1, dtype=torch.int64, device=dev)
        status = torch.zeros(1, dtype=torch.int32, device=dev)
        pc = _col(probe_key)
        _check(lib().ocl_join_probe(self.ctx.handle, ctypes.byref(self._kc), self.ws.data_ptr(), ctypes.byref(pc),
                                    None if oids is None else oids.data_ptr(), None if m is None else m.data_ptr(),
                                    max_rows, int(bool(pk_build)), op.data_ptr(), ob.data_ptr(), out_capacity,
                                    nout.data_ptr(), status.data_ptr(), ws.data_ptr(), sz.value, _stream(stream)))
        return op, ob, nout, status


def hash_join(build_key, probe_key, oids=None, pk_build=False, out_capacity=None):
    """Blocking equi-join: (probe oids, build oids) of all matching pairs, grouped by probe row.
    Grows the output and re-probes once if out_capacity was too small."""
    jb = JoinBuild(build_key)
    for _ in range(2):
        op, ob, nout, st = jb.probe(probe_key, oids=oids, pk_build=pk_build, out_capacity=out_capacity)
        torch.cuda.current_stream(probe_key.device).synchronize()
        s = int(st.item()) or int(jb.status.item())
        n = int(nout.item())
        if s == OCL_ERR_CAPACITY and n > (out_capacity or 0) and int(jb.status.item()) == 0:
            out_capacity = n
            continue
        if s != OCL_OK:
            raise OcelotError(s, f"join device status ({n} pairs)")
        return op[:n], ob[:n]
    raise OcelotError(OCL_ERR_CAPACITY, "join output")


# ---------------------------------------------------------------- a7-a8
def group_aggregate(gids, ngroups, max_groups, vals, aggs, oids=None, m=None, max_rows=None, stream=None):
    """Grouped aggregation over dense gids -> list of per-aggregate outputs [max_groups]."""
    dev = gids.device
    ctx = context(dev)
    max_rows = gids.numel() if max_rows is None else max_rows
    vc = _cols(vals)
    arr, outs = _aggs(aggs, vals, max_groups, dev)
    sz = ctypes.c_size_t()
    _check(lib().ocl_group_aggregate_workspace_size(ctx.handle, max_groups, vc, len(vals), arr, len(aggs),
                                                    ctypes.byref(sz)))
    ws = _workspace(sz.value, dev)
    _check(lib().ocl_group_aggregate(ctx.handle, gids.data_ptr(), None if oids is None else oids.data_ptr(),
                                     None if m is None else m.data_ptr(), max_rows,
                                     None if ngroups is None else ngroups.data_ptr(), max_groups, vc, len(vals), arr,
                                     len(aggs), ws.data_ptr(), sz.value, _stream(stream)))
    return outs


# ---------------------------------------------------------------- a9 fused
class SgaCall:
    """A prepared fused call: ctypes argument block + outputs + workspace, reusable
    across launches (the benchmark times only ``launch``)."""

    def __init__(self, preds, keys, vals, aggs, expected_groups=1024, out_capacity=None, order_by_key=False,
                 bitmap=False, tier=0, host=False, chunk_rows=1 << 24, device=None, key_sorted=False,
                 distributed=0, ctx=None, sync=False):
        """distributed: 0 local, 1 allgather (replicated result), 2 all-to-all (this rank's hash partition),
        over ctx's NCCL communicator (ctx = a Context after attach_nccl, see distributed.attach_nccl).
        sync: size the workspace for ocl_select_group_aggregate_sync (launch_sync, the restart ladder)."""
        cols = [p[0] for p in preds] + list(keys) + list(vals)
        self.host = host
        self.device = torch.device(device) if device is not None else (
            cols[0].device if cols and not host else torch.device("cuda", torch.cuda.current_device()))
        self.ctx = ctx if ctx is not None else context(self.device)
        n = cols[0].numel() if cols else 0
        self.n = n
        self.aggs_spec = aggs
        self.out_capacity = int(out_capacity if out_capacity is not None else max(4 * expected_groups, 16))
        out_dev = "cpu" if host else self.device
        self._pc = _cols([p[0] for p in preds])
        self._pr = (Range * max(len(preds), 1))()
        for i, (c, spec) in enumerate(preds):
            self._pr[i] = _range(spec, c.dtype)
        self._kc = _cols(keys)
        self._vc = _cols(vals)
        self._keep = cols
        outs = [_agg_out(s, vals, self.out_capacity, out_dev) for s in aggs]
        if host:
            outs = [o.pin_memory() for o in outs]
        self._aggs, self.outs = _aggs(aggs, vals, self.out_capacity, out_dev, outs)
        mk = (lambda *a, **k: torch.zeros(*a, **k).pin_memory()) if host else torch.zeros
        self.keys_out = mk(self.out_capacity, dtype=torch.int64, **({} if host else {"device": self.device}))
        self.ngroups = mk(1, dtype=torch.int64, **({} if host else {"device": self.device}))
        self.status = mk(1, dtype=torch.int32, **({} if host else {"device": self.device}))
        self.bitmap = torch.zeros(max((n + 31) // 32, 1), dtype=torch.int32, device=self.device) if bitmap else None
        a = SgaArgs()
        a.pred_cols, a.preds, a.npreds = ctypes.addressof(self._pc), ctypes.addressof(self._pr), len(preds)
        a.nkeys, a.key_cols = len(keys), ctypes.addressof(self._kc)
        a.val_cols, a.nvals = ctypes.addressof(self._vc), len(vals)
        a.naggs, a.aggs = len(aggs), ctypes.addressof(self._aggs)
        a.expected_groups, a.out_capacity = int(expected_groups), self.out_capacity
        a.keys_out, a.ngroups_out = self.keys_out.data_ptr(), self.ngroups.data_ptr()
        a.bitmap_out = self.bitmap.data_ptr() if bitmap else None
        a.dev_status = self.status.data_ptr()
        a.order_by_key, a.tier = int(bool(order_by_key)), int(tier)
        a.key_sorted = int(bool(key_sorted))
        a.distributed = int(distributed)
        self.args = a
        self.chunk_rows = int(chunk_rows)
        sz = ctypes.c_size_t()
        if sync and not host:
            _check(lib().ocl_select_group_aggregate_sync_workspace_size(self.ctx.handle, ctypes.byref(a),
                                                                        ctypes.byref(sz)))
        elif host:
            _check(lib().ocl_select_group_aggregate_host_workspace_size(self.ctx.handle, ctypes.byref(a),
                                                                        self.chunk_rows, ctypes.byref(sz)))
        else:
            _check(lib().ocl_select_group_aggregate_workspace_size(self.ctx.handle, ctypes.byref(a), ctypes.byref(sz)))
        self.ws_bytes = sz.value
        self.ws = _workspace(sz.value, self.device)

    def launch(self, stream=None):
        if self.host:
            _check(lib().ocl_select_group_aggregate_host(self.ctx.handle, ctypes.byref(self.args), self.chunk_rows,
                                                         self.ws.data_ptr(), self.ws_bytes, _stream(stream)))
        else:
            _check(lib().ocl_select_group_aggregate(self.ctx.handle, ctypes.byref(self.args), self.ws.data_ptr(),
                                                    self.ws_bytes, _stream(stream)))

    def launch_sync(self, stream=None):
        """ocl_select_group_aggregate_sync: blocking, restarts with a larger table on overflow.
        Needs sync=True at construction (workspace for the restart ladder)."""
        _check(lib().ocl_select_group_aggregate_sync(self.ctx.handle, ctypes.byref(self.args), self.ws.data_ptr(),
                                                     self.ws_bytes, _stream(stream)))

    def capture(self, stream=None):
        """Record launch() once into a CUDA graph (torch.cuda.CUDAGraph) and return it: replay() re-runs the
        whole fused call (table init, kernels, finalisation) with one launch — for small, launch-bound inputs.
        The graph reuses this call's arguments, workspace and outputs."""
        if self.host:
            raise ValueError("the host-buffer path synchronises inside; it cannot be captured")
        s = stream or torch.cuda.Stream(self.device)
        s.wait_stream(torch.cuda.current_stream(self.device))
        with torch.cuda.stream(s):
            self.launch(s)                                   # warm-up outside the capture (lazy attributes)
        torch.cuda.current_stream(self.device).wait_stream(s)
        g = torch.cuda.CUDAGraph()
        with torch.cuda.graph(g, stream=s):
            self.launch(s)
        return g

    def result(self):
        """Synchronise, check the device status, return (keys[G], [outs[G]]) (host path: CPU tensors)."""
        if not self.host:
            torch.cuda.current_stream(self.device).synchronize()
        st = int(self.status.item())
        if st != OCL_OK:
            raise OcelotError(st, f"device status (G={int(self.ngroups.item())}, capacity {self.out_capacity})")
        G = int(self.ngroups.item())
        return self.keys_out[:G], [o[:G] for o in self.outs]


def select_group_aggregate(preds, keys, vals, aggs, expected_groups=4, out_capacity=None, order_by_key=False,
                           bitmap=False, tier=0, stream=None, max_retries=8, key_sorted=False):
    """Fused select -> group -> aggregate, blocking, with the paper's restart-with-a-larger-table on overflow
    (P:L523-527).  preds = [(column, range_spec)], keys = [column], vals = [column].
    key_sorted=True: the packed key column is sorted -> sort-based grouping, output in key
    order; an unsorted key column raises OcelotError(OCL_ERR_INVALID_ARG).
    Returns (keys_out[G], [outputs[G]], bitmap or None)."""
    # The table restart runs in the library (ocl_select_group_aggregate_sync); only the OUTPUT
    # buffers (caller memory, sized by out_capacity) are re-allocated here when G exceeds them.
    cap = out_capacity
    for _ in range(max_retries):
        call = SgaCall(preds, keys, vals, aggs, expected_groups=expected_groups, out_capacity=cap,
                       order_by_key=order_by_key, bitmap=bitmap, tier=tier, key_sorted=key_sorted, sync=True)
        try:
            call.launch_sync(stream)
            k, o = call.result()
            return k, o, call.bitmap
        except OcelotError as e:
            if e.status != OCL_ERR_CAPACITY:
                raise
            G = int(call.ngroups.item())             # > out_capacity: G (or a lower bound while the table was full)
            cap = max(4 * call.out_capacity, 2 * G)
            expected_groups = max(expected_groups, G)
    raise OcelotError(OCL_ERR_CAPACITY, "hash table still full after retries")


def select_group_aggregate_host(preds, keys, vals, aggs, expected_groups=4, out_capacity=None, order_by_key=False,
                                chunk_rows=1 << 24, tier=0):
    """End-to-end path from HOST (ideally pinned) columns: chunked H2D overlapped with the fused kernel."""
    call = SgaCall(preds, keys, vals, aggs, expected_groups=expected_groups, out_capacity=out_capacity,
                   order_by_key=order_by_key, tier=tier, host=True, chunk_rows=chunk_rows)
    call.launch()
    return call.result()


# ---------------------------------------------------------------- a10 multi-GPU
def partial_row_bytes(call):
    sz = ctypes.c_size_t()
    _check(lib().ocl_partial_row_bytes(ctypes.byref(call.args), ctypes.byref(sz)))
    return sz.value


def sga_partial(call, partial_capacity, stream=None, status=None, out=None):
    """Local fused pass -> (partial rows uint8[cap, row_bytes], count int64[1]) on the device.
    status: an int32[1] device tensor for this step's overflow flag (default: call.status); out: a
    preallocated (rows, count) pair to write into."""
    rb = partial_row_bytes(call)
    if out is None:
        part = torch.empty((max(partial_capacity, 1), rb), dtype=torch.uint8, device=call.device)
        cnt = torch.empty(1, dtype=torch.int64, device=call.device)
    else:
        part, cnt = out
    args = call.args
    if status is not None:
        args = SgaArgs.from_buffer_copy(call.args)
        args.dev_status = status.data_ptr()
    _check(lib().ocl_sga_partial(call.ctx.handle, ctypes.byref(args), part.data_ptr(), partial_capacity,
                                 cnt.data_ptr(), call.ws.data_ptr(), call.ws_bytes, _stream(stream)))
    return part, cnt


def merge_partials(call, partials, counts, nparts, part_capacity, stream=None):
    """Merge ``nparts`` partial tables (back to back) into call's outputs (keys_out, outs, ngroups)."""
    sz = ctypes.c_size_t()
    _check(lib().ocl_merge_partials_workspace_size(call.ctx.handle, ctypes.byref(call.args), nparts, part_capacity,
                                                   ctypes.byref(sz)))
    ws = _workspace(sz.value, call.device)
    _check(lib().ocl_merge_partials(call.ctx.handle, ctypes.byref(call.args), partials.data_ptr(), nparts,
                                    part_capacity, counts.data_ptr(), ws.data_ptr(), sz.value, _stream(stream)))


def route_partials(part, cnt, nparts, stream=None):
    """Hash-route partial rows (uint8[cap, row_bytes], device count int64[1]) to nparts destinations
    -> (rows grouped by destination uint8[cap, row_bytes], per-destination counts int64[nparts])."""
    ctx = context(part.device)
    cap, rb = part.shape
    sz = ctypes.c_size_t()
    _check(lib().ocl_route_partials_workspace_size(ctx.handle, nparts, ctypes.byref(sz)))
    ws = _workspace(sz.value, part.device)
    out = torch.empty_like(part)
    counts = torch.zeros(nparts, dtype=torch.int64, device=part.device)
    _check(lib().ocl_route_partials(ctx.handle, part.data_ptr(), cnt.data_ptr(), cap, rb, nparts, out.data_ptr(),
                                    counts.data_ptr(), ws.data_ptr(), sz.value, _stream(stream)))
    return out, counts


from .distributed import attach_nccl, distributed_select_group_aggregate, shard_range  # noqa: E402,F401
