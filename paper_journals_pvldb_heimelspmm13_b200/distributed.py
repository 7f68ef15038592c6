"""Row-partitioned multi-GPU select -> group -> aggregate.

The paper runs on one device at a time; multi-device execution is its stated
future work.  Here every rank owns a contiguous row range and
runs the fused pass on its shard into a *partial* table of mergeable per-group
states (``ocl_sga_partial``).  Two exchanges (NCCL over NVLink through
``torch.distributed`` — plumbing; the routing and merging run in the library):

* ``allgather`` (few groups): every rank receives all partial tables and merges
  them by key (``ocl_merge_partials``) -> the replicated result.  Latency-bound, no
  host synchronisation for tables up to 1 MB.
* ``alltoall`` (many groups): each partial row is routed to the rank owning its
  key's hash partition (``ocl_route_partials``), ranks exchange only those rows
  (``all_to_all_single`` with per-destination counts), and each rank merges what it
  received -> rank r holds partition r of the groups (``gather_results`` collects
  them).  Each rank receives ~G/P rows instead of (P-1)*G_r — the paper's
  partitioning instead of one global hash table.

AVG is recomputed from the merged SUM and COUNT (never an average of averages).
"""
from __future__ import annotations

import torch
import torch.distributed as dist

# the exchange is sent whole (no host round trip for the max size) below this many bytes per rank
_SMALL_EXCHANGE = 1 << 20


def shard_range(n, rank, world):
    """Contiguous rows [start, start + length) of ``rank``; the remainder goes to the first ranks."""
    base, rem = divmod(n, world)
    start = rank * base + min(rank, rem)
    return start, base + (1 if rank < rem else 0)


def exchange_partials(part, cnt, group=None):
    """Allgather per-rank partial tables.

    part: uint8[cap, row_bytes] (rows >= cnt are padding), cnt: int64[1] valid rows.
    Returns (all_parts uint8[P, cap_x, row_bytes] contiguous, all_counts int64[P], cap_x).
    Works for any backend (NCCL on GPU tensors, gloo on CPU tensors).
    """
    world = dist.get_world_size(group)
    counts = torch.empty(world, dtype=cnt.dtype, device=cnt.device)
    dist.all_gather_into_tensor(counts, cnt.reshape(1), group=group)
    cap, rb = part.shape
    if cap * rb <= _SMALL_EXCHANGE:
        send = part
        cap_x = cap
    else:
        cap_x = max(int(counts.max().item()), 1)     # host sync only for large tables
        send = part[:cap_x].contiguous()
    out = torch.empty((world, cap_x, rb), dtype=part.dtype, device=part.device)
    dist.all_gather_into_tensor(out.view(world * cap_x, rb), send, group=group)
    return out, counts, cap_x


def exchange_routed(rows, counts, group=None):
    """All-to-all of routed partial rows.

    rows: [R, row_bytes] grouped by destination (counts[d] rows for destination d, in
    destination order), counts: int64[P].  Returns (received rows [S, row_bytes], S),
    the rows every rank routed to this one, back to back.  One host synchronisation
    (the split sizes).  Works for any backend (NCCL on GPU tensors, gloo on CPU).
    """
    recv_counts = torch.empty_like(counts)
    dist.all_to_all_single(recv_counts, counts, group=group)
    send = [int(c) for c in counts.tolist()]
    recv = [int(c) for c in recv_counts.tolist()]
    total = sum(recv)
    out = torch.empty((total, rows.shape[1]), dtype=rows.dtype, device=rows.device)
    dist.all_to_all_single(out, rows[:sum(send)].contiguous(), recv, send, group=group)
    return out, total


def distributed_select_group_aggregate(call, partial_capacity=None, group=None, stream=None, mode="auto"):
    """Run ``call`` (an :class:`SgaCall` over this rank's shard) and merge across ranks.

    mode "allgather": the replicated result in ``call.keys_out`` / ``call.outs`` /
    ``call.ngroups``.  mode "alltoall": this rank's hash partition of the groups there
    (see :func:`gather_results`).  "auto" picks allgather for partial tables up to 1 MB.
    """
    from . import merge_partials, partial_row_bytes, route_partials, sga_partial
    cap = call.out_capacity if partial_capacity is None else partial_capacity
    if mode == "auto":
        mode = "allgather" if cap * partial_row_bytes(call) <= _SMALL_EXCHANGE else "alltoall"
    part, cnt = sga_partial(call, cap, stream)
    if mode == "allgather":
        all_parts, counts, cap_x = exchange_partials(part, cnt, group)
        merge_partials(call, all_parts, counts, all_parts.shape[0], cap_x, stream)
    elif mode == "alltoall":
        routed, counts = route_partials(part, cnt, dist.get_world_size(group), stream)
        recv, total = exchange_routed(routed, counts, group)
        recv_cnt = torch.tensor([total], dtype=torch.int64, device=part.device)
        merge_partials(call, recv if total else part[:1], recv_cnt, 1, max(total, 1), stream)
    else:
        raise ValueError(f"mode {mode!r}")
    return call


def gather_results(keys, outs, group=None):
    """Allgather per-rank (keys[G_r], [outs[G_r]]) of an all-to-all merge -> the whole result on every rank
    (ranks' partitions back to back).  One host synchronisation (the largest G_r)."""
    world = dist.get_world_size(group)
    g = torch.tensor([keys.shape[0]], dtype=torch.int64, device=keys.device)
    gs = torch.empty(world, dtype=torch.int64, device=keys.device)
    dist.all_gather_into_tensor(gs, g, group=group)
    sizes = [int(x) for x in gs.tolist()]
    gmax = max(max(sizes), 1)

    def cat(t):
        pad = torch.zeros((gmax,) + tuple(t.shape[1:]), dtype=t.dtype, device=t.device)
        pad[:t.shape[0]] = t
        allp = torch.empty((world * gmax,) + tuple(t.shape[1:]), dtype=t.dtype, device=t.device)
        dist.all_gather_into_tensor(allp, pad, group=group)
        return torch.cat([allp[r * gmax:r * gmax + sizes[r]] for r in range(world)])

    return cat(keys), [cat(o) for o in outs]
