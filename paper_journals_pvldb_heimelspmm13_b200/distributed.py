"""Row-partitioned multi-GPU select -> group -> aggregate.

The paper runs on one device at a time; multi-device execution is its stated
future work.  Every rank owns a contiguous row range and
aggregates its shard into a *partial* table of mergeable per-group states.

Product path — the exchange runs inside the library (``ocl_sga_args.distributed``):
:func:`attach_nccl` gives a :class:`Context` an NCCL communicator
(``ocl_ctx_attach_nccl``; the 128-byte unique id travels over ``torch.distributed`` —
plumbing), and an :class:`SgaCall` built with ``distributed=1`` (allgather: replicated
result) or ``distributed=2`` (hash-partitioned all-to-all: each rank owns a partition of
the groups) runs partial -> NCCL exchange -> merge -> finalise on its stream, with no
host synchronisation (CUDA-graph capturable) and the overflow decision shared by all
ranks.

Portable path (:func:`distributed_select_group_aggregate`) — the same library steps
(``ocl_sga_partial`` / ``ocl_route_partials`` / ``ocl_merge_partials``) with the exchange
done by ``torch.distributed`` collectives, for process groups whose backend is not NCCL
(e.g. gloo: the multi-process tests run it on one GPU).

* ``allgather`` (few groups): every rank receives all partial tables and merges them by
  key -> the replicated result.
* ``alltoall`` (many groups): each partial row is routed to the rank owning its key's
  hash partition, ranks exchange only those rows and merge what they receive -> rank r
  holds partition r of the groups (``gather_results`` collects them).  Each rank
  receives ~G/P rows instead of (P-1)*G_r — the paper's partitioning instead of one
  global hash table.

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


def attach_nccl(device=None, group=None):
    """A new :class:`Context` on ``device`` joined to an NCCL communicator over the ranks of ``group``
    (ocl_nccl_unique_id on rank 0, broadcast over torch.distributed, ocl_ctx_attach_nccl everywhere).
    Collective: every rank of the group calls it."""
    from . import Context, nccl_unique_id
    rank, world = dist.get_rank(group), dist.get_world_size(group)
    obj = [nccl_unique_id() if rank == 0 else None]
    dist.broadcast_object_list(obj, src=dist.get_global_rank(group, 0) if group is not None else 0, group=group)
    ctx = Context(device)
    ctx.attach_nccl(obj[0], rank, world)
    return ctx


def exchange_partials(part, cnt, cap, group=None):
    """Allgather per-rank partial tables.

    part: uint8[cap, row_bytes] (rows >= cnt are padding), cnt: int64[1] valid rows (<= cap: the caller
    has checked overflow).  Returns (all_parts uint8[P, cap_x, row_bytes] contiguous, all_counts int64[P],
    cap_x).  Works for any backend (NCCL on GPU tensors, gloo on CPU or GPU tensors).
    """
    world = dist.get_world_size(group)
    counts = torch.empty(world, dtype=cnt.dtype, device=cnt.device)
    dist.all_gather_into_tensor(counts, cnt.reshape(1), group=group)
    rb = part.shape[1]
    if cap * rb <= _SMALL_EXCHANGE:
        cap_x = cap
    else:
        cap_x = min(max(int(counts.max().item()), 1), cap)     # host sync only for large tables
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
    """Portable multi-rank path: run ``call`` (an :class:`SgaCall` over this rank's shard, distributed=0)
    and merge across ranks with torch.distributed collectives.

    mode "allgather": the replicated result in ``call.keys_out`` / ``call.outs`` / ``call.ngroups``.
    mode "alltoall": this rank's hash partition of the groups there (see :func:`gather_results`).
    "auto" picks allgather for partial tables up to 1 MB.  Every rank must use the same mode and capacity.

    Overflow: the partial step reports into its own status word; every rank contributes
    (status != 0 or rows > capacity) to an all-reduce MAX, so all ranks agree and raise
    OcelotError(OCL_ERR_CAPACITY) together instead of merging truncated tables (the caller
    restarts with a larger expected_groups / partial_capacity).
    """
    from . import OCL_ERR_CAPACITY, OcelotError, merge_partials, partial_row_bytes, route_partials, sga_partial
    cap = call.out_capacity if partial_capacity is None else partial_capacity
    if mode == "auto":
        mode = "allgather" if cap * partial_row_bytes(call) <= _SMALL_EXCHANGE else "alltoall"
    pstatus = torch.zeros(1, dtype=torch.int32, device=call.device)
    part, cnt = sga_partial(call, cap, stream, status=pstatus)
    flag = ((pstatus != 0) | (cnt > cap)).to(torch.int64)
    dist.all_reduce(flag, op=dist.ReduceOp.MAX, group=group)
    if int(flag.item()):
        raise OcelotError(OCL_ERR_CAPACITY, f"a rank's partial table overflowed (capacity {cap}): restart larger")
    if mode == "allgather":
        all_parts, counts, cap_x = exchange_partials(part, cnt, cap, group)
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
