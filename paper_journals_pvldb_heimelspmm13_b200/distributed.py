"""Row-partitioned multi-GPU select -> group -> aggregate.

The paper runs on one device at a time; multi-device execution is its stated
future work.  Here every rank owns a contiguous row range,
runs the fused pass on its shard into a *partial* table of mergeable per-group
states (``ocl_sga_partial``), the ranks exchange those tables with an allgather
(NCCL over NVLink through ``torch.distributed`` — plumbing) and every rank merges
all of them by key (``ocl_merge_partials``), so the result is replicated.  AVG is
recomputed from the merged SUM and COUNT (never an average of averages).
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


def distributed_select_group_aggregate(call, partial_capacity=None, group=None, stream=None):
    """Run ``call`` (an :class:`SgaCall` over this rank's shard) and merge across ranks.

    Leaves the replicated result in ``call.keys_out`` / ``call.outs`` / ``call.ngroups``.
    """
    from . import merge_partials, sga_partial
    cap = call.out_capacity if partial_capacity is None else partial_capacity
    part, cnt = sga_partial(call, cap, stream)
    all_parts, counts, cap_x = exchange_partials(part, cnt, group)
    merge_partials(call, all_parts, counts, all_parts.shape[0], cap_x, stream)
    return call
