"""Generator checks (host side): shard consistency and the distribution facts of
SURVEY.md §8(c)/(d) (sanity checks on the synthetic workload, not parity)."""
import numpy as np

import datagen


def test_shard_consistency():
    n = 10000
    full = datagen.lineitem_host(n, 123, fields=datagen.LINEITEM_INT_FIELDS + datagen.LINEITEM_F64_FIELDS)
    part = datagen.lineitem_host(3000, 123, fields=datagen.LINEITEM_INT_FIELDS + datagen.LINEITEM_F64_FIELDS,
                                 row0=4000, n_total=n)
    for f, a in part.items():
        assert (a == full[f][4000:7000]).all(), f


def test_lineitem_distribution():
    n = 280000
    li = datagen.lineitem_host(n, datagen.BASE_SEED + 2)
    # Q1 selectivity 1 - 4095/291126 = 0.985934; correlated per order, so tolerance over orders
    sel = (li["shipdate"] <= datagen.Q1_SHIP_CUTOFF).mean()
    p = 1 - 4095 / 291126
    sigma_orders = np.sqrt(p * (1 - p) / (n / 4)) * 2.0
    assert abs(sel - p) < 5 * sigma_orders
    assert abs(li["quantity"].mean() / 100 - 25.5) < 0.2
    assert abs(li["discount"].mean() - 5.0) < 0.05
    assert abs(li["tax"].mean() - 4.0) < 0.05
    assert set(np.unique(li["returnflag"]).tolist()) == {ord("A"), ord("N"), ord("R")}
    assert set(np.unique(li["linestatus"]).tolist()) == {ord("F"), ord("O")}
    # line counts: 7 orders per 28 rows -> n/4 orders, orderkeys sparse (8 of every 32)
    ok = np.unique(li["orderkey"])
    assert len(ok) == n // 4
    assert ((ok - 1) % 32 < 8).all()
    # max per-row charge stays far below 2^63 (s12)
    charge = li["extendedprice"] * (100 - li["discount"]) * (100 + li["tax"])
    assert charge.max() < 2**40


def test_f64_is_decimal_over_100():
    li = datagen.lineitem_host(1000, 7, fields=("quantity", "quantity_f", "tax", "tax_f"))
    assert (li["quantity_f"] == li["quantity"] / 100.0).all()
    assert (li["tax_f"] == li["tax"] / 100.0).all()


def test_shuffled_is_permutation():
    n = 5000
    a = datagen.lineitem_host(n, 9, fields=("orderkey", "quantity"))
    b = datagen.lineitem_host(n, 9, fields=("orderkey", "quantity"), shuffled=True)
    pa = sorted(zip(a["orderkey"].tolist(), a["quantity"].tolist()))
    pb = sorted(zip(b["orderkey"].tolist(), b["quantity"].tolist()))
    assert pa == pb and not (a["orderkey"] == b["orderkey"]).all()


def test_sweep_zipf():
    G = 1 << 10
    sw = datagen.sweep_host(200000, 5, G, s=1.5)
    vals, cnt = np.unique(sw["key"], return_counts=True)
    top = cnt.max() / cnt.sum()
    H = sum((i + 1) ** -1.5 for i in range(G))
    assert abs(top - 1 / H) < 0.01                     # ~38% of rows on the top key
    uni = datagen.sweep_host(200000, 5, 16, s=0.0)
    assert len(np.unique(uni["key"])) == 16
    assert (uni["p"] >= 0).all() and (uni["p"] < 10**6).all()
