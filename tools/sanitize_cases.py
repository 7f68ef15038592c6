"""One small call of every kernel family of libocelot_b200, for compute-sanitizer (`make sanitize`).

Sizes are small (the sanitizers slow kernels down ~100x) but each call spans several CTAs, a
ragged tail and, for the pipelined kernels, several ring stages.  Every result is checked
against the oracle so a sanitizer run is also a parity run.  Exit code 0 = all results equal.

    compute-sanitizer --tool memcheck|racecheck|synccheck --error-exitcode 1 python tools/sanitize_cases.py
"""
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import numpy as np  # noqa: E402
import torch  # noqa: E402

import datagen  # noqa: E402
import oracle  # noqa: E402
import paper_journals_pvldb_heimelspmm13_b200 as ocl  # noqa: E402
from tests._common import Q1_AGGS, Q1_AGGS_F64, assert_results_equal, by_key  # noqa: E402

DEV = torch.device("cuda", 0)
ONLY = set(sys.argv[1:])


def dev(a):
    return torch.from_numpy(np.ascontiguousarray(a)).to(DEV)


def case(name):
    def wrap(fn):
        if not ONLY or name in ONLY:
            fn()
            torch.cuda.synchronize()
            print(f"ok {name}", flush=True)
        return fn
    return wrap


def check_sga(preds, keys, vals, aggs, **kw):
    k, outs, _ = ocl.select_group_aggregate([(dev(c), s) for c, s in preds], [dev(c) for c in keys],
                                            [dev(c) for c in vals], aggs, **kw)
    rk, routs = oracle.sga(preds, keys, vals, aggs)
    dts = [c.dtype for c in vals]
    assert_results_equal(by_key(k.cpu().numpy(), [o.cpu().numpy() for o in outs], aggs, dts),
                         by_key(rk, routs, aggs, dts), aggs, dts)
    return ocl.last_kernel(ocl.context(DEV))


li = datagen.lineitem_host(40_000, datagen.BASE_SEED + 1,
                           fields=datagen.LINEITEM_INT_FIELDS + datagen.LINEITEM_F64_FIELDS)
Q1P = [(li["shipdate"], {"hi": 10471})]
Q1K = [li["returnflag"], li["linestatus"]]
Q1V = [li["quantity"], li["extendedprice"], li["discount"], li["tax"]]
Q1VF = [li["quantity_f"], li["extendedprice_f"], li["discount_f"], li["tax_f"]]
C5AGGS = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "min", "a": 0}, {"op": "max", "a": 0}]
sw = datagen.sweep_host(70_001, datagen.BASE_SEED + 5, 300, s=1.0)


@case("select_compact_gather")
def _():
    x = li["shipdate"]
    bm = ocl.select_bitmap(dev(x), {"lo": 9000, "hi": 10000})
    assert np.array_equal(bm.cpu().numpy().view(np.uint32), oracle.select(x, {"lo": 9000, "hi": 10000}))
    b2 = ocl.bitmap_combine("and", bm, ocl.select_bitmap(dev(x), {"hi": 9500}), len(x))
    oids, m = ocl.prefix_compact(b2, len(x))
    ref = oracle.compact(oracle.bitmap_combine("and", oracle.select(x, {"lo": 9000, "hi": 10000}),
                                               oracle.select(x, {"hi": 9500}), len(x)), len(x))
    mm = int(m.item())
    assert np.array_equal(oids[:mm].cpu().numpy().view(np.uint32), ref)
    g = ocl.gather(dev(li["quantity"]), oids[:mm])
    assert np.array_equal(g.cpu().numpy(), li["quantity"][ref])


@case("group_build_aggregate")
def _():
    keys = [sw["key"]]
    for scheme in ("b200", "paper"):
        gids, kout, ng, st = ocl.group_build([dev(keys[0])], expected_groups=600, scheme=scheme)
        torch.cuda.synchronize()
        assert int(st.item()) == 0 and int(ng.item()) == len(np.unique(keys[0]))
    gids = np.searchsorted(np.unique(sw["key"]), sw["key"]).astype(np.int32)
    G = int(gids.max()) + 1
    got = ocl.group_aggregate(dev(gids), None, G, [dev(sw["v"])], C5AGGS)
    ref = oracle.aggregate(gids, G, [sw["v"]], C5AGGS)
    for o, r in zip(got, ref):
        assert np.array_equal(o[:G].cpu().numpy().reshape(r.shape), r)


@case("fused_q1_bulk_priv")
def _():
    assert "k_sga_bulk<Sig Q1 int64>" in check_sga(Q1P, Q1K, Q1V, Q1_AGGS, expected_groups=4)
    assert "k_sga_bulk<Sig Q1 fp64>" in check_sga(Q1P, Q1K, Q1VF, Q1_AGGS_F64, expected_groups=4)
    assert "Q1+MINMAX" in check_sga(Q1P, Q1K, Q1V, Q1_AGGS + [{"op": "min", "a": 0}, {"op": "max", "a": 1}],
                                    expected_groups=4)
    small = [(c[:300], s) for c, s in Q1P]
    assert "k_sga_priv" in check_sga(small, [c[:300] for c in Q1K], [c[:300] for c in Q1V], Q1_AGGS,
                                     expected_groups=4)


@case("fused_groupby_tiers")
def _():
    p = [(sw["p"], {"hi": 699_999})]
    assert "4 private slots" in check_sga(p, [sw["key"] % 3], [sw["v"]], C5AGGS, expected_groups=4)
    assert "CTA table" in check_sga(p, [sw["key"]], [sw["v"]], C5AGGS, expected_groups=300)
    for tier in (1, 2, 3, 4):          # generic register tier, HBM tier, dynamic shape, CTA table
        check_sga(p, [sw["key"]], [sw["v"]], C5AGGS, expected_groups=300, tier=tier)
    check_sga(p, [sw["key"]], [sw["v"]], C5AGGS, expected_groups=2000, tier=5)   # hash-partitioned


@case("partitioned_two_level")
def _():
    # 256 partitions: level-1 scatter into per-block ranges, level-2 direct-map tiles; ~1.8x the
    # expected groups, so shared tables overflow into lazily zeroed HBM regions
    rng = np.random.default_rng(29)
    n, E = 1 << 20, 1 << 18
    key = rng.integers(0, int(1.8 * E), n).astype(np.int64) * 7919
    x = rng.integers(-10**6, 10**6, n).astype(np.int64)
    assert "partitioned" in check_sga([], [key], [x], C5AGGS, expected_groups=E, tier=5, out_capacity=4 * E)


@case("fused_select_compact_gather")
def _():
    os.environ["OCL_SPARSE_PCT"] = "100"      # k_sga_sparse whenever the sample selects < 100 %
    try:
        p = [(sw["p"], {"hi": 19_999})]
        assert "CTA table" in check_sga(p, [sw["key"]], [sw["v"]], C5AGGS, expected_groups=300)
        assert "4 private slots" in check_sga(p, [sw["key"] % 3], [sw["v"]], C5AGGS, expected_groups=4)
        assert "k_sga_bulk<Sig Q1 int64>" in check_sga([(li["shipdate"], {"hi": 8200})], Q1K, Q1V, Q1_AGGS,
                                                       expected_groups=4)
    finally:
        del os.environ["OCL_SPARSE_PCT"]


@case("sorted_radix_tier6")
def _():
    lo = datagen.lineitem_host(50_000, datagen.BASE_SEED + 3)
    k, outs, _ = ocl.select_group_aggregate([], [dev(lo["orderkey"])], [dev(lo["quantity"])], C5AGGS,
                                            expected_groups=20_000, out_capacity=20_000, key_sorted=True)
    rk, routs = oracle.sga([], [lo["orderkey"]], [lo["quantity"]], C5AGGS, order_by_key=True)
    assert np.array_equal(k.cpu().numpy(), rk)
    rng = np.random.default_rng(1)
    perm = rng.permutation(len(lo["orderkey"]))
    check_sga([], [lo["orderkey"][perm]], [lo["quantity"][perm]], C5AGGS, expected_groups=20_000,
              out_capacity=20_000, tier=6)
    ks, pl, rows = ocl.radix_sort([dev(lo["orderkey"][perm])], payload=dev(lo["quantity"][perm]), rowids=True)
    order = np.argsort(lo["orderkey"][perm].view(np.uint64), kind="stable")
    assert np.array_equal(rows.cpu().numpy().view(np.uint32), order.astype(np.uint32))


@case("join")
def _():
    rng = np.random.default_rng(2)
    build = rng.permutation(20_000).astype(np.int64) * 3
    probe = rng.integers(0, 70_000, 60_000).astype(np.int64)
    for pk in (True, False):
        b = build if pk else np.concatenate([build, build[:500]])
        po, bo = ocl.hash_join(dev(b), dev(probe), pk_build=pk, out_capacity=200_000)
        rp, rb = oracle.hash_join(b, probe)
        assert len(po) == len(rp)
        got = sorted(zip(po.cpu().numpy().view(np.uint32).tolist(), bo.cpu().numpy().view(np.uint32).tolist()))
        assert got == sorted(zip(rp.tolist(), rb.tolist()))


@case("partials_route_merge")
def _():
    from paper_journals_pvldb_heimelspmm13_b200.distributed import shard_range
    n, P = len(sw["key"]), 3
    parts, counts = [], []
    for r in range(P):
        s0, ln = shard_range(n, r, P)
        call = ocl.SgaCall([], [dev(sw["key"][s0:s0 + ln])], [dev(sw["v"][s0:s0 + ln])], C5AGGS,
                           expected_groups=300, out_capacity=600)
        part, cnt = ocl.sga_partial(call, 600)
        routed, rc = ocl.route_partials(part, cnt, 2)
        parts.append(part)
        counts.append(cnt)
    call = ocl.SgaCall([], [dev(sw["key"])], [dev(sw["v"])], C5AGGS, expected_groups=300, out_capacity=600)
    ocl.merge_partials(call, torch.stack(parts).contiguous(), torch.cat(counts), P, 600)
    k, outs = call.result()
    rk, routs = oracle.sga([], [sw["key"]], [sw["v"]], C5AGGS)
    assert_results_equal(by_key(k.cpu().numpy(), [o.cpu().numpy() for o in outs], C5AGGS, [np.int64]),
                         by_key(rk, routs, C5AGGS, [np.int64]), C5AGGS, [np.int64])


@case("distributed_nccl_world1")
def _():
    ctx = ocl.Context(0)
    ctx.attach_nccl(ocl.nccl_unique_id(), 0, 1)
    for mode in (1, 2):
        call = ocl.SgaCall([(dev(c), s) for c, s in Q1P], [dev(c) for c in Q1K], [dev(c) for c in Q1V], Q1_AGGS,
                           expected_groups=4, out_capacity=16, distributed=mode, ctx=ctx)
        call.launch()
        k, outs = call.result()
        rk, routs = oracle.sga(Q1P, Q1K, Q1V, Q1_AGGS)
        dts = [c.dtype for c in Q1V]
        assert_results_equal(by_key(k.cpu().numpy(), [o.cpu().numpy() for o in outs], Q1_AGGS, dts),
                             by_key(rk, routs, Q1_AGGS, dts), Q1_AGGS, dts)


@case("host_path")
def _():
    t = lambda c: torch.from_numpy(c).pin_memory()
    k, outs = ocl.select_group_aggregate_host([(t(c), s) for c, s in Q1P], [t(c) for c in Q1K], [t(c) for c in Q1V],
                                              Q1_AGGS, expected_groups=4, chunk_rows=1 << 14)
    rk, routs = oracle.sga(Q1P, Q1K, Q1V, Q1_AGGS)
    dts = [c.dtype for c in Q1V]
    assert_results_equal(by_key(k.numpy(), [o.numpy() for o in outs], Q1_AGGS, dts),
                         by_key(rk, routs, Q1_AGGS, dts), Q1_AGGS, dts)

print("all sanitizer cases ok")
