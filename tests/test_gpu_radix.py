"""Radix sort (§4.1.3) and the sort-based grouping tier
(tier 6: radix sort, then the sorted-input path) through the C ABI vs the oracle / library routines.

A stable sort by key is unique, so keys, payloads and row ids are compared exactly against
numpy's stable argsort (a library routine) of the packed key."""
import numpy as np
import pytest
import torch

import datagen
import oracle
from tests._common import assert_results_equal, by_key

pytestmark = pytest.mark.gpu

ocl = pytest.importorskip("paper_journals_pvldb_heimelspmm13_b200")
DEV = torch.device("cuda", 0)


def dev(a):
    return torch.from_numpy(np.ascontiguousarray(a)).to(DEV)


@pytest.mark.parametrize("n", [1, 31, 4095, 4096, 4097, 100003, (1 << 21) + 5])
@pytest.mark.parametrize("dom", [1, 200, 1 << 26, 1 << 62])
def test_radix_sort_i64(n, dom):
    rng = np.random.default_rng(n + dom % 1000)
    keys = rng.integers(0, dom, n).astype(np.int64)
    pay = rng.integers(-10**12, 10**12, n).astype(np.int64)
    ko, po, ro = ocl.radix_sort([dev(keys)], payload=dev(pay), rowids=True)
    perm = np.argsort(keys.view(np.uint64), kind="stable")
    assert np.array_equal(ko.cpu().numpy(), keys[perm])
    assert np.array_equal(po.cpu().numpy(), pay[perm])
    assert np.array_equal(ro.cpu().numpy().view(np.uint32), perm.astype(np.uint32))


def test_radix_sort_packed_keys_and_negatives():
    rng = np.random.default_rng(2)
    n = 50000
    a = rng.integers(0, 256, n).astype(np.uint8)
    b = rng.integers(-5, 5, n).astype(np.int32)                      # packed: raw 32-bit pattern
    ko, _, ro = ocl.radix_sort([dev(a), dev(b)], rowids=True)
    packed = (a.astype(np.uint64) << np.uint64(32)) | b.view(np.uint32).astype(np.uint64)
    perm = np.argsort(packed, kind="stable")
    assert np.array_equal(ko.cpu().numpy().view(np.uint64), packed[perm])
    assert np.array_equal(ro.cpu().numpy().view(np.uint32), perm.astype(np.uint32))
    neg = rng.integers(-10**15, 10**15, n).astype(np.int64)          # full 64-bit range: 8 passes
    ko, _, _ = ocl.radix_sort([dev(neg)])
    assert np.array_equal(ko.cpu().numpy().view(np.uint64), np.sort(neg.view(np.uint64), kind="stable"))


@pytest.mark.parametrize("shuffled", [True, False])
def test_tier6_sort_group_c3_shape(shuffled):
    """C3 shape (GROUP BY orderkey, COUNT/SUM/MIN/MAX(quantity)) in shuffled and dbgen order."""
    n = 1_000_003
    li = datagen.lineitem_host(n, datagen.BASE_SEED + 3, shuffled=shuffled)
    aggs = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "min", "a": 0}, {"op": "max", "a": 0},
            {"op": "avg", "a": 0}]
    k, outs, _ = ocl.select_group_aggregate([], [dev(li["orderkey"])], [dev(li["quantity"])], aggs,
                                            expected_groups=n // 4, out_capacity=n // 2, tier=6)
    rk, routs = oracle.sga([], [li["orderkey"]], [li["quantity"]], aggs, order_by_key=True)
    assert np.array_equal(k.cpu().numpy(), rk)                          # key order
    dts = [np.int64]
    assert_results_equal(by_key(k.cpu().numpy(), [o.cpu().numpy() for o in outs], aggs, dts),
                         by_key(rk, routs, aggs, dts), aggs, dts)


def test_tier6_generic_and_f64():
    rng = np.random.default_rng(8)
    n = 300000
    a = rng.integers(0, 50, n).astype(np.uint8)
    b = rng.integers(0, 7, n).astype(np.uint8)
    f = rng.integers(0, 10**6, n).astype(np.float64) / 100.0
    aggs = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "avg", "a": 0}, {"op": "min", "a": 0}, {"op": "max", "a": 0}]
    k, outs, _ = ocl.select_group_aggregate([], [dev(a), dev(b)], [dev(f)], aggs, out_capacity=1000, tier=6)
    rk, routs = oracle.sga([], [a, b], [f], aggs, order_by_key=True)
    assert np.array_equal(k.cpu().numpy(), rk)
    assert_results_equal(by_key(k.cpu().numpy(), [o.cpu().numpy() for o in outs], aggs, [np.float64]),
                         by_key(rk, routs, aggs, [np.float64]), aggs, [np.float64])
    with pytest.raises(ocl.OcelotError, match="UNSUPPORTED"):
        ocl.select_group_aggregate([(dev(b), {"hi": 3})], [dev(a)], [dev(f)], aggs, tier=6)


def test_radix_and_tier6_edges():
    """n = 0 and n = 1; all keys equal (one run over every tile); keys at the top of the 64-bit range."""
    e = np.zeros(0, np.int64)
    ko, po, ro = ocl.radix_sort([dev(e)], payload=dev(e), rowids=True)
    assert ko.numel() == 0 and po.numel() == 0 and ro.numel() == 0
    aggs = [{"op": "count"}, {"op": "sum", "a": 0}]
    k, outs, _ = ocl.select_group_aggregate([], [dev(e)], [dev(e)], aggs, tier=6)
    assert k.numel() == 0
    one = np.array([7], np.int64)
    k, outs, _ = ocl.select_group_aggregate([], [dev(one)], [dev(one)], aggs, tier=6)
    assert k.cpu().tolist() == [7] and outs[0].cpu().tolist() == [1]
    n = 100000
    same = np.full(n, 123456789, np.int64)
    v = np.arange(n, dtype=np.int64)
    k, outs, _ = ocl.select_group_aggregate([], [dev(same)], [dev(v)], aggs, out_capacity=4, tier=6)
    assert k.cpu().tolist() == [123456789] and outs[0].cpu().tolist() == [n]
    assert int(outs[1][0, 0].item()) == n * (n - 1) // 2
    top = (np.uint64(2**64 - 1) - np.arange(1000, dtype=np.uint64) % 7).view(np.int64)
    ko, _, ro = ocl.radix_sort([dev(top)], rowids=True)
    perm = np.argsort(top.view(np.uint64), kind="stable")
    assert np.array_equal(ko.cpu().numpy(), top[perm])
    assert np.array_equal(ro.cpu().numpy().view(np.uint32), perm.astype(np.uint32))
