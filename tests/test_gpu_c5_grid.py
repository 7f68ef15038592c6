"""Config C5 correctness grid ("Oracle correctness covers every C5 point at n = 2^22"):
G in {2^2, 2^4, ..., 2^24} x Zipf s in {0, 1.0, 1.5} x selectivity in {1 %, 50 %, 100 %} = 108 points
of WHERE p < T GROUP BY key: COUNT, SUM, MIN, MAX(v), through the library's automatic tier choice
(expected_groups = G, as the benchmark and tools/sweep_c5.py call it), each compared with the oracle
group by group (integers bit-exact)."""
import numpy as np
import pytest
import torch

import datagen
import oracle

pytestmark = [pytest.mark.gpu, pytest.mark.slow]

ocl = pytest.importorskip("paper_journals_pvldb_heimelspmm13_b200")
N = 1 << 22
AGGS = [{"op": "count"}, {"op": "sum", "a": 0}, {"op": "min", "a": 0}, {"op": "max", "a": 0}]


def _sorted_result(keys, outs):
    k = np.asarray(keys).view(np.uint64)
    order = np.argsort(k, kind="stable")
    return k[order], [np.asarray(o)[order] for o in outs]


@pytest.mark.parametrize("lg", [2, 4, 6, 8, 10, 12, 14, 16, 18, 20, 22, 24])
@pytest.mark.parametrize("s", [0.0, 1.0, 1.5])
def test_c5_grid(lg, s):
    G = 1 << lg
    sw = datagen.sweep_host(N, datagen.BASE_SEED + 5, G, s=s)
    dev = torch.device("cuda", 0)
    p, key, v = (torch.from_numpy(sw[f]).to(dev) for f in ("p", "key", "v"))
    for sel in (0.01, 0.5, 1.0):
        T = int(round(sel * 10**6))
        pred = {"hi": T - 1}
        gk, gouts, _ = ocl.select_group_aggregate([(p, pred)], [key], [v], AGGS, expected_groups=G,
                                                  out_capacity=max(16, 2 * G))
        kernel = ocl.last_kernel(ocl.context(dev))
        rk, routs = oracle.sga([(sw["p"], pred)], [sw["key"]], [sw["v"]], AGGS)
        a_k, a_o = _sorted_result(gk.cpu().numpy(), [o.cpu().numpy() for o in gouts])
        b_k, b_o = _sorted_result(rk, routs)
        assert np.array_equal(a_k, b_k), (G, s, sel, kernel, len(a_k), len(b_k))
        for i, (x, y) in enumerate(zip(a_o, b_o)):
            assert np.array_equal(x.reshape(y.shape), y), (G, s, sel, kernel, AGGS[i])
