"""Multi-GPU host logic on CPU: row sharding and the partial-table allgather, world size 2 over gloo.

The CUDA merge kernel is covered on the GPU by test_gpu_parity.py::test_sharded_partials_merge
(fake exchange).  Here the partial tables are produced by the oracle on each rank's shard, sent
through exchange_partials (the same function the NCCL path uses) and merged by key in Python;
the result must equal the oracle over all rows (sharding changes no integer bit).
"""
import os
import socket

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

from paper_journals_pvldb_heimelspmm13_b200.distributed import exchange_partials, shard_range


@pytest.mark.parametrize("n,world", [(0, 2), (1, 2), (7, 3), (1000, 8), (600_000_001, 8)])
def test_shard_range_partition(n, world):
    spans = [shard_range(n, r, world) for r in range(world)]
    pos = 0
    for s, ln in spans:
        assert s == pos and ln >= 0
        pos += ln
    assert pos == n
    lens = [ln for _, ln in spans]
    assert max(lens) - min(lens) <= 1


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, n, q):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        import datagen
        import oracle
        start, ln = shard_range(n, rank, world)
        li = datagen.lineitem_host(ln, 77, row0=start, n_total=n)
        vals = [li["quantity"], li["extendedprice"], li["discount"]]
        aggs = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "min", "a": 1}, {"op": "max", "a": 2}]
        keys, outs = oracle.sga([(li["shipdate"], {"hi": 10471})], [li["returnflag"], li["linestatus"]], vals, aggs)
        # partial rows: key, count, sum lo, sum hi, min, max  (6 x int64 = 48 bytes)
        G = len(keys)
        cap = 8
        rows = np.zeros((cap, 6), np.int64)
        rows[:G, 0] = keys
        rows[:G, 1] = outs[0]
        rows[:G, 2:4] = outs[1].view(np.int64).reshape(G, 2)
        rows[:G, 4] = outs[2]
        rows[:G, 5] = outs[3]
        part = torch.from_numpy(rows.view(np.uint8).reshape(cap, 48).copy())
        cnt = torch.tensor([G], dtype=torch.int64)
        allp, counts, cap_x = exchange_partials(part, cnt, cap)
        assert allp.shape == (world, cap_x, 48)
        merged = {}
        for r in range(world):
            t = allp[r].numpy().view(np.int64).reshape(cap_x, 6)
            for j in range(int(counts[r])):
                k, c, lo, hi, mn, mx = (int(x) for x in t[j])
                s = ((hi & 0xFFFFFFFFFFFFFFFF) << 64) | (lo & 0xFFFFFFFFFFFFFFFF)
                s = s - (1 << 128) if s >= 1 << 127 else s
                m = merged.setdefault(k, [0, 0, None, None])
                m[0] += c
                m[1] += s
                m[2] = mn if m[2] is None else min(m[2], mn)
                m[3] = mx if m[3] is None else max(m[3], mx)
        if rank == 0:
            q.put(merged)
    finally:
        dist.destroy_process_group()


def test_gloo_allgather_merge_equals_oracle():
    import datagen
    import oracle
    n, world = 200_003, 2
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, world, port, n, q)) for r in range(world)]
    for p in procs:
        p.start()
    merged = q.get(timeout=300)
    for p in procs:
        p.join(timeout=120)
        assert p.exitcode == 0
    li = datagen.lineitem_host(n, 77)
    vals = [li["quantity"], li["extendedprice"], li["discount"]]
    aggs = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "min", "a": 1}, {"op": "max", "a": 2}]
    keys, outs = oracle.sga([(li["shipdate"], {"hi": 10471})], [li["returnflag"], li["linestatus"]], vals, aggs)
    ref = {}
    sums = outs[1].view(np.int64).reshape(len(keys), 2)
    for i, k in enumerate(keys.tolist()):
        s = ((int(sums[i, 1]) & 0xFFFFFFFFFFFFFFFF) << 64) | (int(sums[i, 0]) & 0xFFFFFFFFFFFFFFFF)
        ref[k] = [int(outs[0][i]), s, int(outs[2][i]), int(outs[3][i])]
    assert merged == ref


# ---------------------------------------------------------------- overflow agreement
def _overflow_worker(rank, world, port, bad_rank, how, q):
    """distributed_select_group_aggregate's host logic with the library steps stubbed (no GPU here): one
    rank's partial overflows -> every rank raises OCL_ERR_CAPACITY before any exchange of truncated tables."""
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        import paper_journals_pvldb_heimelspmm13_b200 as pkg
        from paper_journals_pvldb_heimelspmm13_b200.distributed import distributed_select_group_aggregate
        merged = []

        def fake_partial(call, cap, stream=None, status=None, out=None):
            cnt = torch.tensor([cap + 5 if (rank == bad_rank and how == "count") else 2], dtype=torch.int64)
            if rank == bad_rank and how == "status":
                status[0] = pkg.OCL_ERR_CAPACITY
            return torch.zeros((cap, 48), dtype=torch.uint8), cnt

        pkg.sga_partial = fake_partial
        pkg.partial_row_bytes = lambda call: 48
        pkg.merge_partials = lambda call, allp, counts, nparts, cap, stream=None: merged.append(counts.tolist())

        class Call:
            out_capacity = 16
            device = torch.device("cpu")

        try:
            distributed_select_group_aggregate(Call(), mode="allgather")
            q.put((rank, "ok", merged))
        except pkg.OcelotError as e:
            q.put((rank, "capacity" if e.status == pkg.OCL_ERR_CAPACITY else "other", merged))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("bad_rank,how", [(-1, "none"), (1, "status"), (0, "count")])
def test_gloo_overflow_agreement(bad_rank, how):
    world = 2
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_overflow_worker, args=(r, world, port, bad_rank, how, q)) for r in range(world)]
    for p in procs:
        p.start()
    res = sorted(q.get(timeout=300) for _ in range(world))
    for p in procs:
        p.join(timeout=120)
        assert p.exitcode == 0
    if bad_rank < 0:
        assert [r[1] for r in res] == ["ok", "ok"] and all(r[2] == [[2, 2]] for r in res)
    else:
        assert [r[1] for r in res] == ["capacity", "capacity"] and all(r[2] == [] for r in res)


# ---------------------------------------------------------------- all-to-all (hash-routed) exchange, NEXT-2
def _fmix64(k):
    k = np.asarray(k, dtype=np.uint64).copy()
    k ^= k >> np.uint64(33)
    k *= np.uint64(0xFF51AFD7ED558CCD)
    k ^= k >> np.uint64(33)
    k *= np.uint64(0xC4CEB9FE1A85EC53)
    k ^= k >> np.uint64(33)
    return k


def route_of(keys, P):
    """Destination rank of a key (the ABI's definition, include/ocelot_b200.h ocl_route_partials)."""
    return ((_fmix64(keys) & np.uint64(0xFFFFFFFF)) * np.uint64(P)) >> np.uint64(32)


def _a2a_worker(rank, world, port, q):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        from paper_journals_pvldb_heimelspmm13_b200.distributed import exchange_routed, gather_results
        rng = np.random.default_rng(100 + rank)
        nrows = 5000 + 1000 * rank
        rows = np.zeros((nrows, 4), np.int64)                       # 32-byte partial rows: key, count, 2 states
        rows[:, 0] = rng.integers(0, 1 << 40, nrows)
        rows[:, 1] = rank + 1
        rows[:, 2] = np.arange(nrows)
        dest = route_of(rows[:, 0], world).astype(np.int64)
        order = np.argsort(dest, kind="stable")                    # grouped by destination (what the kernel does)
        routed = torch.from_numpy(rows[order].view(np.uint8).reshape(nrows, 32).copy())
        counts = torch.from_numpy(np.bincount(dest, minlength=world).astype(np.int64))
        recv, total = exchange_routed(routed, counts)
        got = recv.numpy().view(np.int64).reshape(total, 4)
        assert (route_of(got[:, 0], world).astype(np.int64) == rank).all()   # only this rank's partition
        keys = torch.from_numpy(got[:, 0].copy())
        allk, allo = gather_results(keys, [torch.from_numpy(got[:, 1:].copy())])
        if rank == 0:
            q.put((sorted(map(tuple, np.concatenate([allk.numpy()[:, None], allo[0].numpy()], 1).tolist()))))
    finally:
        dist.destroy_process_group()


def test_gloo_alltoall_routed_exchange():
    """Rows routed by key hash reach exactly their owner; the gathered union equals everything sent."""
    world = 3
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_a2a_worker, args=(r, world, port, q)) for r in range(world)]
    for p in procs:
        p.start()
    got = q.get(timeout=300)
    for p in procs:
        p.join(timeout=120)
        assert p.exitcode == 0
    sent = []
    for rank in range(world):
        rng = np.random.default_rng(100 + rank)
        nrows = 5000 + 1000 * rank
        k = rng.integers(0, 1 << 40, nrows)
        sent += [(int(k[i]), rank + 1, i, 0) for i in range(nrows)]
    assert got == sorted(sent)
