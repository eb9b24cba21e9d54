"""NEXT-1 inputs and oracle: TPC-C Delivery as in-place updates.

Pins, none of which use the oracle's own update code:
  * SQLite executes the TPC-C Delivery SQL (MIN(o_id) of the undelivered orders per district,
    UPDATE orders / UPDATE order_line) from the same random inputs; the updated columns, in
    rowid order, must equal ``oracle.apply_updates`` of chgen's row-update sets, and the CH
    queries SQLite runs on the updated tables must equal the oracle's on the updated snapshot;
  * draining every district delivers every line: no NULL delivery date remains, so Q1 with an
    early cutoff counts every order_line row;
  * the previous snapshot is unchanged (copy-on-write: a later epoch never alters an earlier).
"""
import numpy as np
import pytest

import chgen
import oracle
from chref import (Q18_HAVING, sqlite_column, sqlite_delivery, sqlite_load, sqlite_q1,
                   sqlite_q18, sqlite_q3, sqlite_q6, visible)

NULL = np.iinfo(np.int64).min


def _state(tables, sc):
    st = chgen.DeliveryState(districts=sc.districts)
    st.add(tables["orders"], 0, 0)
    return st


@pytest.mark.parametrize("mode", ["spread", "strict"])
def test_delivery_updates_match_sqlite(mode):
    sc = chgen.TINY
    W = 2
    t = chgen.generate(1, W + 1, seed=5, mode=mode, scale=sc, with_item=False)
    # a NewOrder delta appended first, so deliveries cross from loaded into appended orders
    no = chgen.NewOrderState(1, W + 1, scale=sc)
    item = chgen.generate_item(5, sc)
    delta = chgen.neworder_batch(no, 12, seed=5, batch=0, item=item)
    st = _state(t, sc)
    st.add(delta["orders"], len(t["orders"]["o_id"]), len(t["order_line"]["ol_o_id"]))
    for tb in ("orders", "order_line"):
        t[tb] = {c: np.concatenate([t[tb][c], delta[tb][c]]) for c in t[tb]}
    db = sqlite_load(t)
    snap = t
    clock = chgen.TS_2025 + 7 * chgen.DAY_US
    for b in range(4):
        w, carrier = chgen.delivery_inputs(3, seed=5, batch=b, w_lo=1, w_hi=W + 1)
        upd = chgen.delivery_batch(st, w, carrier, clock)
        for k in range(len(w)):
            sqlite_delivery(db, int(w[k]), int(carrier[k]), clock + (k + 1) * 1000, sc.districts)
        clock += len(w) * 1000
        prev = snap
        prev_copy = {tb: {c: v.copy() for c, v in cols.items()} for tb, cols in prev.items()}
        snap = oracle.apply_updates(snap, upd)
        for tb in prev:  # the earlier snapshot is untouched
            for c in prev[tb]:
                assert np.array_equal(prev[tb][c], prev_copy[tb][c])
        assert sqlite_column(db, "order_line", "ol_delivery_d", NULL) == snap["order_line"]["ol_delivery_d"].tolist()
        assert sqlite_column(db, "orders", "o_carrier_id", -1) == snap["orders"]["o_carrier_id"].tolist()
        assert len(np.unique(upd["order_line"]["ol_delivery_d"][0])) == len(upd["order_line"]["ol_delivery_d"][0])
        # the CH queries over the updated snapshot
        hi = clock + chgen.DAY_US
        r6 = oracle.q6(snap, chgen.TS_1995, hi, 1, 100000)
        assert r6["revenue"] == sqlite_q6(db, chgen.TS_1995, hi, 1, 100000)
        r1 = oracle.q1(snap, chgen.TS_2025)
        want1 = sqlite_q1(db, chgen.TS_2025)
        assert r1["ol_number"].tolist() == [r[0] for r in want1]
        assert r1["count_order"].tolist() == [r[5] for r in want1]
        assert r1["sum_amount"].tolist() == [r[2] for r in want1]
        r18 = oracle.q18(snap, Q18_HAVING)
        assert len(r18["o_id"]) == len(sqlite_q18(db, Q18_HAVING))


def test_draining_delivers_every_line():
    sc = chgen.TINY
    t = chgen.generate(1, 3, seed=9, scale=sc, with_item=False)
    st = _state(t, sc)
    undelivered_lines = int((t["order_line"]["ol_delivery_d"] == NULL).sum())
    assert st.undelivered() == int((t["orders"]["o_carrier_id"] == -1).sum()) > 0
    snap, b, n_upd = t, 0, 0
    while st.undelivered():
        w, carrier = chgen.delivery_inputs(4, seed=9, batch=b, w_lo=1, w_hi=3)
        upd = chgen.delivery_batch(st, w, carrier, chgen.TS_2025 + b * 10**6)
        n_upd += len(upd["order_line"]["ol_delivery_d"][0])
        snap = oracle.apply_updates(snap, upd)
        b += 1
    assert n_upd == undelivered_lines
    assert not (snap["order_line"]["ol_delivery_d"] == NULL).any()
    assert not (snap["orders"]["o_carrier_id"] == -1).any()
    r1 = oracle.q1(snap, chgen.TS_1995 - 1)
    assert int(r1["count_order"].sum()) == len(snap["order_line"]["ol_o_id"])


def test_delivery_takes_oldest_order_per_district():
    sc = chgen.TINY
    t = chgen.generate(1, 2, seed=3, scale=sc, with_item=False)
    st = _state(t, sc)
    upd = chgen.delivery_batch(st, np.array([1], np.int32), np.array([7], np.int32), chgen.TS_2025)
    rows, vals = upd["orders"]["o_carrier_id"]
    o = t["orders"]
    assert o["o_id"][rows].tolist() == [sc.delivered_below] * sc.districts
    assert o["o_d_id"][rows].tolist() == list(range(1, sc.districts + 1))
    assert vals.tolist() == [7] * sc.districts
    lrows, lvals = upd["order_line"]["ol_delivery_d"]
    ol = t["order_line"]
    assert set(zip(ol["ol_d_id"][lrows].tolist(), ol["ol_o_id"][lrows].tolist())) == \
        {(d, sc.delivered_below) for d in range(1, sc.districts + 1)}
    assert len(lrows) == int(o["o_ol_cnt"][rows].sum())
    assert (lvals == chgen.TS_2025 + 1000).all()


def test_delivery_deletes_new_order_rows_like_sqlite():
    """Delivery's DELETE FROM new_order as a tombstone update (R35): SQLite executes
    the DELETE; the new_order rows without a tombstone in chgen's updated snapshot must be exactly
    SQLite's remaining rows (rowid order), and CH Q3 — which joins new_order — must agree between
    SQLite and the oracle on the visible snapshot, epoch after epoch, across a NewOrder delta."""
    sc = chgen.TINY
    W = 2
    t = chgen.generate(1, W + 1, seed=15, scale=sc)
    item = t.pop("item")
    st = chgen.DeliveryState(districts=sc.districts)
    st.add(t["orders"], 0, 0, 0)  # generated new_order rows list the undelivered orders in order
    no = chgen.NewOrderState(1, W + 1, scale=sc)
    delta = chgen.neworder_batch(no, 10, seed=15, batch=0, item=item)
    st.add(delta["orders"], len(t["orders"]["o_id"]), len(t["order_line"]["ol_o_id"]),
           len(t["new_order"]["no_o_id"]))
    for tb in ("orders", "order_line", "new_order"):
        t[tb] = {c: np.concatenate([t[tb][c], delta[tb][c]]) for c in t[tb]}
    db = sqlite_load(t)
    snap = t
    clock = chgen.TS_2025 + 3 * chgen.DAY_US
    entry_lo = chgen.TS_1995
    deleted = 0
    for b in range(5):
        w, carrier = chgen.delivery_inputs(2, seed=15, batch=b, w_lo=1, w_hi=W + 1)
        upd = chgen.delivery_batch(st, w, carrier, clock)
        for k in range(len(w)):
            sqlite_delivery(db, int(w[k]), int(carrier[k]), clock + (k + 1) * 1000, sc.districts)
        clock += len(w) * 1000
        snap = oracle.apply_updates(snap, upd)
        deleted += len(upd["new_order"]["no_deleted"][0])
        vis = visible(snap)["new_order"]
        got = db.execute("SELECT no_w_id, no_d_id, no_o_id FROM new_order ORDER BY rowid").fetchall()
        assert got == list(zip(vis["no_w_id"].tolist(), vis["no_d_id"].tolist(), vis["no_o_id"].tolist()))
        assert int(snap["new_order"]["no_deleted"].sum()) == deleted > 0
        want = sqlite_q3(db, entry_lo, "")
        got3 = oracle.q3(visible(snap), entry_lo, b"")
        rows = list(zip(got3["ol_o_id"].tolist(), got3["ol_w_id"].tolist(), got3["ol_d_id"].tolist(),
                        got3["revenue"].tolist(), got3["o_entry_d"].tolist()))
        assert len(rows) > 0
        # SQLite breaks ORDER BY ties arbitrarily: the ordered sort keys and the row set must match
        assert [(r[3], r[4]) for r in rows] == [(r[3], r[4]) for r in want]
        assert sorted(rows) == sorted(tuple(r) for r in want)
