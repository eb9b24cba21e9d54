"""T0: the seeded input generator (shared input module; holds no query arithmetic)."""
import numpy as np
import pytest

import chgen


def test_population_shape_and_domains():
    t = chgen.generate(1, 3, seed=1, mode="spread")
    o, ol, c = t["orders"], t["order_line"], t["customer"]
    assert len(o["o_id"]) == 2 * 10 * 3000 and len(c["c_id"]) == 2 * 10 * 3000
    assert len(ol["ol_w_id"]) == int(o["o_ol_cnt"].sum())
    assert o["o_ol_cnt"].min() >= 5 and o["o_ol_cnt"].max() <= 15
    # PKs unique
    ko = o["o_w_id"].astype(np.int64) << 40 | o["o_d_id"].astype(np.int64) << 32 | o["o_id"]
    assert len(np.unique(ko)) == len(ko)
    kc = c["c_w_id"].astype(np.int64) << 40 | c["c_d_id"].astype(np.int64) << 32 | c["c_id"]
    assert len(np.unique(kc)) == len(kc)
    # o_c_id is a permutation of 1..3000 per district
    for w in (1, 2):
        for d in (1, 10):
            m = (o["o_w_id"] == w) & (o["o_d_id"] == d)
            assert sorted(o["o_c_id"][m].tolist()) == list(range(1, 3001))
    undelivered = ol["ol_o_id"] >= 2101
    assert (ol["ol_delivery_d"][undelivered] == chgen.NULL_TS).all()
    assert (ol["ol_delivery_d"][~undelivered] != chgen.NULL_TS).all()
    assert ol["ol_quantity"].min() >= 1 and ol["ol_quantity"].max() <= 10
    assert ol["ol_amount"].min() >= 1 and ol["ol_amount"].max() <= 999_999
    assert c["c_last"].min() >= 0 and c["c_last"].max() <= 999
    assert (c["c_last"][c["c_id"] <= 1000] == c["c_id"][c["c_id"] <= 1000] - 1).all()


@pytest.mark.parametrize("world", [2, 3])
def test_shards_are_byte_identical_slices(world):
    W = 4
    whole = chgen.generate(1, W + 1, seed=3, with_item=False)
    for lo, hi in chgen.warehouse_ranges(W, world):
        part = chgen.generate(lo, hi, seed=3, with_item=False)
        for tname, cols in part.items():
            wcol = {"order_line": "ol_w_id", "orders": "o_w_id", "customer": "c_w_id",
                    "new_order": "no_w_id"}[tname]
            m = (whole[tname][wcol] >= lo) & (whole[tname][wcol] < hi)
            for cname, arr in cols.items():
                assert np.array_equal(arr, whole[tname][cname][m]), (tname, cname)


def test_warehouse_ranges_cover():
    for W, n in [(100, 8), (7, 3), (1, 1), (1000, 8)]:
        r = chgen.warehouse_ranges(W, n)
        assert r[0][0] == 1 and r[-1][1] == W + 1
        assert all(a[1] == b[0] for a, b in zip(r, r[1:]))
        sizes = [hi - lo for lo, hi in r]
        assert max(sizes) - min(sizes) <= 1


def test_neworder_delta_appends_fresh_orders():
    st = chgen.NewOrderState(1, 3)
    d = chgen.neworder_delta(st, 20, seed=1, batch=0)
    assert len(d["orders"]["o_id"]) == 20
    assert (d["orders"]["o_id"] >= 3001).all()
    assert len(d["order_line"]["ol_o_id"]) == int(d["orders"]["o_ol_cnt"].sum())
    assert (d["order_line"]["ol_delivery_d"] == chgen.NULL_TS).all()


def test_new_order_and_c_state():
    """new_order = the undelivered orders (TPC-C 4.3.3.1: o_id 2101..3000 per district, matching
    orders with a NULL carrier, TPC-C consistency condition 5); c_state 2 characters of the
    a-string alphabet, its device encoding = (byte0 << 8) | byte1; NewOrder deltas insert one
    new_order row per order."""
    t = chgen.generate(1, 3, seed=2)
    o, no, c = t["orders"], t["new_order"], t["customer"]
    assert len(no["no_o_id"]) == 2 * 10 * 900
    und = o["o_carrier_id"] == -1
    assert set(zip(no["no_w_id"].tolist(), no["no_d_id"].tolist(), no["no_o_id"].tolist())) == \
        set(zip(o["o_w_id"][und].tolist(), o["o_d_id"][und].tolist(), o["o_id"][und].tolist()))
    assert no["no_o_id"].min() == 2101 and no["no_o_id"].max() == 3000
    st = [bytes(x) for x in c["c_state"]]
    assert all(len(x) == 2 and x.isalnum() for x in st)
    assert [x[0] << 8 | x[1] for x in st] == c["c_state_p2"].tolist()
    d = chgen.neworder_batch(chgen.NewOrderState(1, 3), 7, seed=1, batch=0)
    assert d["new_order"]["no_o_id"].tolist() == d["orders"]["o_id"].tolist()
