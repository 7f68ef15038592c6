"""Equi hash join (§4.1.5) through the C ABI vs the CPU oracle.

Pairs are grouped by probe row in ascending probe order on both sides; a probe row's partners
come in unspecified order from the GPU, so they are compared as sorted (probe, build) pairs —
with the probe order itself checked exactly.
"""
import numpy as np
import pytest
import torch

import oracle

pytestmark = pytest.mark.gpu

ocl = pytest.importorskip("paper_journals_pvldb_heimelspmm13_b200")
DEV = torch.device("cuda", 0)


def dev(a):
    return torch.from_numpy(np.ascontiguousarray(a)).to(DEV)


def _check(build, probe, oids=None, pk_build=False):
    op, ob = ocl.hash_join(dev(build), dev(probe), oids=None if oids is None else dev(oids.view(np.int32)),
                           pk_build=pk_build)
    gp = op.cpu().numpy().view(np.uint32)
    gb = ob.cpu().numpy().view(np.uint32)
    rp, rb = oracle.hash_join(build, probe, oids)
    assert len(gp) == len(rp)
    assert np.array_equal(gp, rp)                                      # grouped by probe row, probe order
    gi, ri = np.lexsort((gb, gp)), np.lexsort((rb, rp))                 # partners compared as sets
    assert np.array_equal(gb[gi], rb[ri])
    return len(gp)


@pytest.mark.parametrize("n_build,n_probe", [(0, 100), (1, 1), (100, 0), (1000, 3000), (70001, 500003),
                                             (1 << 20, (1 << 21) + 17)])
def test_join_pk_fk(n_build, n_probe):
    """PK-FK: unique build keys, foreign keys with dangling values; direct (pk_build) and two-step."""
    rng = np.random.default_rng(n_build + n_probe)
    pk = (rng.permutation(max(n_build, 1))[:n_build].astype(np.int64) * 2654435761) % (1 << 40)
    fk = rng.choice(pk, n_probe) if n_build else rng.integers(0, 10, n_probe).astype(np.int64)
    fk[::7] = (1 << 41) + np.arange(len(fk[::7]))                      # no partner
    for pkb in (True, False):
        _check(pk, fk, pk_build=pkb)
    oids = np.flatnonzero(rng.random(n_probe) < 0.3).astype(np.uint32)
    _check(pk, fk, oids=oids, pk_build=True)


@pytest.mark.parametrize("dtype,dom", [(np.int32, 50), (np.int64, 5000), (np.uint8, 256), (np.int64, 3)])
def test_join_many_to_many(dtype, dom):
    """Duplicate build keys: the paper's two-step count / prefix sum / write join."""
    rng = np.random.default_rng(dom)
    build = rng.integers(-dom // 2 if dtype != np.uint8 else 0, dom // 2 + 1 if dtype != np.uint8 else 256,
                         20000).astype(dtype)
    probe = rng.integers(-dom // 2 if dtype != np.uint8 else 0, dom // 2 + 1 if dtype != np.uint8 else 256,
                         30001).astype(dtype)
    assert _check(build, probe) > 0


def test_join_edge_cases():
    keys = np.array([-1, 5, -1, 7], np.int64)                          # key ~0 (all ones) on both sides
    _check(keys, np.array([-1, 7, 8, -1], np.int64))
    dup = np.array([1, 2, 2, 3], np.int64)
    jb = ocl.JoinBuild(dev(dup))
    _, _, _, st = jb.probe(dev(np.array([2, 3], np.int64)), pk_build=True)
    torch.cuda.synchronize()
    assert int(st.item()) == ocl.OCL_ERR_INVALID_ARG                  # not a key column
    _, _, n, st = jb.probe(dev(np.array([2, 2, 2], np.int64)), out_capacity=2)
    torch.cuda.synchronize()
    assert int(st.item()) == ocl.OCL_ERR_CAPACITY and int(n.item()) == 6
    with pytest.raises(ocl.OcelotError):
        jb.probe(dev(np.array([2], np.int32)))                          # dtypes differ


@pytest.mark.parametrize("pk_build", [True, False])
def test_join_dense_domain(pk_build):
    """Build keys in a dense domain (range < 4 x rows, unique): the direct-array build; TPC-H orders keys
    (8 of every 32 used) against lineitem-like foreign keys, probes below / above the range, and a dense
    domain with a repeated key (falls back to the hash table)."""
    import datagen
    nb = 70007
    pk = datagen.orders_keys(nb)                                       # sparse(o): dense within 4x
    rng = np.random.default_rng(11)
    fk = np.sort(rng.choice(pk, 300001))                              # clustered probe (dbgen order)
    fk[::13] = pk.min() - 1 - (np.arange(len(fk[::13])) % 5)           # below the range
    fk[5::17] = pk.max() + 1 + (np.arange(len(fk[5::17])) % 7)         # above the range
    _check(pk, fk, pk_build=pk_build)
    oids = np.flatnonzero(rng.random(len(fk)) < 0.5).astype(np.uint32)
    _check(pk, fk, oids=oids, pk_build=pk_build)
    dup = pk.copy()
    dup[100] = dup[200]                                               # one repeated key
    if pk_build:
        jb = ocl.JoinBuild(dev(dup))
        _, _, _, st = jb.probe(dev(fk), pk_build=True, out_capacity=2 * len(fk))
        torch.cuda.synchronize()
        assert int(st.item()) == ocl.OCL_ERR_INVALID_ARG
    else:
        _check(dup, fk, pk_build=False)
