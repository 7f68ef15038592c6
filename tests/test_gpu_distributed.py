"""Multi-GPU path through the library (the paper's future work, PAPER.md
L1240-1248): ocl_ctx_attach_nccl + ocl_sga_args.distributed (partial -> NCCL exchange -> merge ->
finalise inside the library, on the call's stream), ocl_select_group_aggregate_sync (the restart of
P:L523-527 in C), and the portable torch.distributed path across processes.

The box has one GPU and NCCL refuses two ranks on one device, so the NCCL path runs on a world-size-1
communicator (every step executes: the allgather / send-recv of headers and tables, the header check,
the merge and the finalisation); the multi-rank composition of the library steps runs across two
processes sharing the GPU through the gloo backend (portable path).  Results vs the oracle over all
rows (SURVEY §8(c) rules).
"""
import os
import socket

import numpy as np
import pytest
import torch
import torch.multiprocessing as mp

import datagen
import oracle
from tests._common import Q1_AGGS, assert_results_equal, by_key

pytestmark = pytest.mark.gpu

ocl = pytest.importorskip("paper_journals_pvldb_heimelspmm13_b200")
DEV = torch.device("cuda", 0)


def dev(a):
    return torch.from_numpy(np.ascontiguousarray(a)).to(DEV)


@pytest.fixture(scope="module")
def nccl_ctx():
    ctx = ocl.Context(0)
    ctx.attach_nccl(ocl.nccl_unique_id(), 0, 1)
    assert ctx.nccl_rank == (0, 1)
    return ctx


def _q1(n, seed):
    li = datagen.lineitem_host(n, seed)
    vals = [li["quantity"], li["extendedprice"], li["discount"], li["tax"]]
    return [(li["shipdate"], {"hi": 10471})], [li["returnflag"], li["linestatus"]], vals, Q1_AGGS


def _compare(call, preds, keys, vals, aggs, order_by_key=False):
    k, outs = call.result()
    rk, routs = oracle.sga(preds, keys, vals, aggs, order_by_key=order_by_key)
    dts = [c.dtype for c in vals]
    if order_by_key:
        assert k.cpu().numpy().tolist() == rk.tolist()
    assert_results_equal(by_key(k.cpu().numpy(), [o.cpu().numpy() for o in outs], aggs, dts),
                         by_key(rk, routs, aggs, dts), aggs, dts)


@pytest.mark.parametrize("mode", [1, 2])
@pytest.mark.parametrize("n", [0, 1000, 1_000_003])
def test_nccl_q1(nccl_ctx, mode, n):
    """Q1 (4 groups) through partial -> NCCL allgather / all-to-all -> merge -> ORDER BY key."""
    p, k, v, a = _q1(n, datagen.BASE_SEED + 4)
    call = ocl.SgaCall([(dev(c), s) for c, s in p], [dev(c) for c in k], [dev(c) for c in v], a,
                       expected_groups=4, out_capacity=16, order_by_key=True, distributed=mode, ctx=nccl_ctx)
    call.launch()
    _compare(call, p, k, v, a, order_by_key=True)


@pytest.mark.parametrize("mode", [1, 2])
@pytest.mark.parametrize("G", [5000, 300_000])
def test_nccl_many_groups(nccl_ctx, mode, G):
    """Many groups (hash-partitioned local tier above 1024 expected groups), COUNT/SUM/MIN/MAX + fp64 AVG."""
    n = (1 << 21) + 5
    sw = datagen.sweep_host(n, datagen.BASE_SEED + 5, G, s=1.0, f64=True)
    preds = [(sw["p"], {"hi": 699_999})]
    aggs = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "min", "a": 0}, {"op": "max", "a": 0},
            {"op": "avg", "a": 1}]
    call = ocl.SgaCall([(dev(c), s) for c, s in preds], [dev(sw["key"])], [dev(sw["v"]), dev(sw["v_f"])], aggs,
                       expected_groups=G, out_capacity=2 * G, distributed=mode, ctx=nccl_ctx)
    call.launch()
    _compare(call, preds, [sw["key"]], [sw["v"], sw["v_f"]], aggs)


def test_nccl_sorted_path(nccl_ctx):
    """The sorted-input local step feeding the exchange."""
    li = datagen.lineitem_host(400_000, datagen.BASE_SEED + 3)
    aggs = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "min", "a": 0}, {"op": "max", "a": 0}]
    call = ocl.SgaCall([], [dev(li["orderkey"])], [dev(li["quantity"])], aggs, expected_groups=110_000,
                       out_capacity=110_000, key_sorted=True, distributed=1, ctx=nccl_ctx)
    call.launch()
    _compare(call, [], [li["orderkey"]], [li["quantity"]], aggs)


def test_nccl_graph_capture(nccl_ctx):
    """The whole distributed call (local pass, NCCL collectives, merge, finalise) as one CUDA graph."""
    p, k, v, a = _q1(60_000, datagen.BASE_SEED + 1)
    call = ocl.SgaCall([(dev(c), s) for c, s in p], [dev(c) for c in k], [dev(c) for c in v], a,
                       expected_groups=4, out_capacity=16, order_by_key=True, distributed=1, ctx=nccl_ctx)
    g = call.capture()
    for _ in range(3):
        call.outs[0].zero_()
        g.replay()
        _compare(call, p, k, v, a, order_by_key=True)


@pytest.mark.parametrize("distributed", [0, 1])
def test_sync_restart(nccl_ctx, distributed):
    """ocl_select_group_aggregate_sync: expected_groups far too small -> the library restarts with a larger
    table until the result fits; G > out_capacity -> OCL_ERR_CAPACITY with G reported."""
    n = 200_000
    rng = np.random.default_rng(3)
    key = rng.integers(0, 30_000, n).astype(np.int64)
    x = rng.integers(-1000, 1000, n).astype(np.int64)
    aggs = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "max", "a": 0}]
    for tier in (0, 2):
        call = ocl.SgaCall([], [dev(key)], [dev(x)], aggs, expected_groups=4, out_capacity=40_000, tier=tier,
                           sync=True, distributed=distributed, ctx=nccl_ctx)
        call.launch_sync()
        _compare(call, [], [key], [x], aggs)
    call = ocl.SgaCall([], [dev(key)], [dev(x)], aggs, expected_groups=4, out_capacity=1000, sync=True,
                       distributed=distributed, ctx=nccl_ctx)
    with pytest.raises(ocl.OcelotError) as e:
        call.launch_sync()
    assert e.value.status == ocl.OCL_ERR_CAPACITY
    assert int(call.ngroups.item()) > 1000


def test_nccl_overflow_reported(nccl_ctx):
    """A partial table larger than out_capacity: every rank skips the merge and reports OCL_ERR_CAPACITY."""
    n = 100_000
    key = np.arange(n, dtype=np.int64) % 5000
    call = ocl.SgaCall([], [dev(key)], [dev(key)], [{"op": "count"}], expected_groups=8192, out_capacity=1000,
                       distributed=1, ctx=nccl_ctx)
    call.launch()
    torch.cuda.synchronize()
    assert int(call.status.item()) == ocl.OCL_ERR_CAPACITY


def test_distributed_needs_communicator():
    x = dev(np.arange(10, dtype=np.int64))
    with pytest.raises(ocl.OcelotError) as e:
        ocl.SgaCall([], [x], [x], [{"op": "count"}], expected_groups=16, distributed=1, ctx=ocl.Context(0))
    assert e.value.status == ocl.OCL_ERR_INVALID_ARG


# ---------------------------------------------------------------- two processes, one GPU (gloo)
def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _gloo_worker(rank, world, port, n, mode, q):
    import torch.distributed as dist
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        import paper_journals_pvldb_heimelspmm13_b200 as ocl_
        from paper_journals_pvldb_heimelspmm13_b200.distributed import (distributed_select_group_aggregate,
                                                                          gather_results, shard_range)
        d = torch.device("cuda", 0)
        s0, ln = shard_range(n, rank, world)
        sw = datagen.sweep_host(ln, datagen.BASE_SEED + 5, 20_000, s=0.0, row0=s0)
        aggs = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "min", "a": 0}, {"op": "max", "a": 0}]
        t = lambda a: torch.from_numpy(np.ascontiguousarray(a)).to(d)
        call = ocl_.SgaCall([(t(sw["p"]), {"hi": 499_999})], [t(sw["key"])], [t(sw["v"])], aggs,
                            expected_groups=20_000, out_capacity=40_000)
        distributed_select_group_aggregate(call, mode=mode)
        k, outs = call.result()
        if mode == "alltoall":
            k, outs = gather_results(k, outs)
        q.put((rank, k.cpu().numpy(), [o.cpu().numpy() for o in outs]))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("mode", ["allgather", "alltoall"])
def test_two_process_portable_path(mode):
    """Product partial -> torch.distributed exchange -> product merge across two processes on cuda:0."""
    n, world = 1_000_003, 2
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_gloo_worker, args=(r, world, port, n, mode, q)) for r in range(world)]
    for p in procs:
        p.start()
    res = sorted((q.get(timeout=600) for _ in range(world)), key=lambda r: r[0])
    for p in procs:
        p.join(timeout=120)
        assert p.exitcode == 0
    sw = datagen.sweep_host(n, datagen.BASE_SEED + 5, 20_000, s=0.0)
    aggs = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "min", "a": 0}, {"op": "max", "a": 0}]
    rk, routs = oracle.sga([(sw["p"], {"hi": 499_999})], [sw["key"]], [sw["v"]], aggs)
    dts = [np.int64]
    for _, k, outs in res:                   # every rank holds the whole result
        assert_results_equal(by_key(k, outs, aggs, dts), by_key(rk, routs, aggs, dts), aggs, dts)
