"""GPU parity of in-place updates (TPC-C Delivery, copy-on-write epochs).

Every epoch's Q1 / Q6 / Q18 through the C ABI must equal the oracle on the host snapshot of that
epoch (``oracle.apply_updates`` of the same row-update sets, pinned to SQLite's Delivery SQL in
test_delivery_oracle.py). Covered: steady-state page catch-up, whole-column copies, appends and
updates in one epoch, queries racing refreshes (each result matches the epoch it reports), I32 /
I64 columns, key-column updates (zone maps widen; duplicate keys are detected), errors, and the
BASELINE full size (W=100).
"""
import threading

import numpy as np
import pytest

import chgen
import oracle
from chref import Q1_CUTOFF, Q6_D_HI, Q6_D_LO, Q6_Q_HI, Q6_Q_LO, Q18_HAVING
from test_gpu_parity import Loader, assert_q1, assert_q6, assert_q18

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module")
def h():
    import paper_conf_cidr_appuswamykpa17_b200 as mod
    return mod


def _hot_updates(h, upd):
    """Keep the updates of columns the hot path loads (o_carrier_id is not one of them)."""
    hot = {}
    for plan in h.HOT_PATH_PLANS:
        for t, cols in h.plan_columns()[plan].items():
            hot.setdefault(t, set()).update(cols)
    return {t: {c: v for c, v in cols.items() if c in hot.get(t, ())} for t, cols in upd.items()}


def _concat(a, b):
    return {c: np.concatenate([a[c], b[c]]) for c in a}


def check_epoch(L, snap, clock):
    """Q6 over a window that includes the Delivery timestamps, Q1 at the CH cutoff and at the
    start of the Delivery clock (counts only lines delivered by the updates), Q18."""
    hi = clock + chgen.DAY_US
    assert_q6(L.q(6, [Q6_D_LO, hi, Q6_Q_LO, Q6_Q_HI]), oracle.q6(snap, Q6_D_LO, hi, Q6_Q_LO, Q6_Q_HI))
    assert_q6(L.q(6), oracle.q6(snap, Q6_D_LO, Q6_D_HI, Q6_Q_LO, Q6_Q_HI))
    assert_q1(L.q(1), oracle.q1(snap, Q1_CUTOFF))
    assert_q1(L.q(1, [chgen.TS_2025]), oracle.q1(snap, chgen.TS_2025))
    assert_q18(L.q(18), oracle.q18(snap, Q18_HAVING))


class Mix:
    """Host side of a NewOrder + Delivery mix: per epoch, a NewOrder delta appended and the
    Delivery row updates (which may deliver orders appended in the same epoch)."""

    def __init__(self, h, W, seed, mode="spread"):
        self.h, self.W, self.seed = h, W, seed
        self.snap = chgen.generate(1, W + 1, seed=seed, mode=mode)
        self.item = self.snap.pop("item")
        self.no = chgen.NewOrderState(1, W + 1)
        self.dl = chgen.DeliveryState()
        self.dl.add(self.snap["orders"], 0, 0)
        self.clock = chgen.TS_2025 + 30 * chgen.DAY_US
        self.b = 0

    def step(self, n_neworder, n_delivery):
        s = self.snap
        n_o, n_ol = len(s["orders"]["o_id"]), len(s["order_line"]["ol_o_id"])
        delta = chgen.neworder_batch(self.no, n_neworder, seed=self.seed, batch=self.b, item=self.item)
        self.dl.add(delta["orders"], n_o, n_ol)
        w, carrier = chgen.delivery_inputs(n_delivery, seed=self.seed, batch=self.b, w_lo=1, w_hi=self.W + 1)
        upd = chgen.delivery_batch(self.dl, w, carrier, self.clock)
        self.clock += (n_delivery + 1) * 1000
        self.b += 1
        grown = {"orders": _concat(s["orders"], delta["orders"]),
                 "order_line": _concat(s["order_line"], delta["order_line"]),
                 "customer": s["customer"]}
        self.snap = oracle.apply_updates(grown, upd)
        hot = self.h.hot_path_tables({**delta, "customer": s["customer"]})
        hot.pop("customer")
        return hot, _hot_updates(self.h, upd), {"orders": n_o, "order_line": n_ol}


def test_delivery_epochs_parity(h):
    e = h.h2tap_open(0)
    try:
        m = Mix(h, W=3, seed=51)
        h.h2tap_load_snapshot(e, h.hot_path_tables(m.snap), 1)
        L = Loader(h, e)
        L.epoch = 1
        check_epoch(L, m.snap, m.clock)
        for k in range(6):
            hot, upd, first = m.step(n_neworder=300, n_delivery=40 + 30 * k)
            L.epoch += 1
            h.h2tap_refresh(e, hot, upd, L.epoch, first_row=first)
            check_epoch(L, m.snap, m.clock)
            st = h.h2tap_get_store_stats(e)
            assert st["published_epoch"] == L.epoch
            if k == 0:
                assert st["cow_full_copies"] == 1      # first update: no shadow yet
            else:
                assert st["cow_full_copies"] == 1      # steady state: page catch-up only
                assert st["cow_pages_copied"] > 0
        assert st["rows_updated"] > 0
        assert st["last_update_ms"] > 0
    finally:
        h.h2tap_close(e)


def test_updates_only_and_full_copy_when_shadow_is_busy(h):
    """Updates without appends; back-to-back async refreshes (the shadow may still be read by a
    pending / published epoch -> whole-column copy); parity after each publish."""
    e = h.h2tap_open(0)
    try:
        m = Mix(h, W=2, seed=52)
        h.h2tap_load_snapshot(e, h.hot_path_tables(m.snap), 1)
        L = Loader(h, e)
        L.epoch = 1
        for k in range(4):
            w, carrier = chgen.delivery_inputs(25, seed=52, batch=100 + k, w_lo=1, w_hi=3)
            upd = chgen.delivery_batch(m.dl, w, carrier, m.clock)
            m.clock += 26_000
            m.snap = oracle.apply_updates(m.snap, upd)
            L.epoch += 1
            h.h2tap_refresh(e, None, _hot_updates(h, upd), L.epoch, flags=h.H2TAP_LOAD_ASYNC)
        assert h.h2tap_sync(e) == L.epoch
        check_epoch(L, m.snap, m.clock)
        st = h.h2tap_get_store_stats(e)
        assert st["cow_full_copies"] >= 1 and st["refreshes"] == 5
    finally:
        h.h2tap_close(e)


def test_queries_racing_update_refreshes(h):
    """A query thread runs while the main thread publishes update epochs: every result must be
    the oracle's answer for exactly the epoch the result reports (old epochs stay intact)."""
    e = h.h2tap_open(0)
    try:
        m = Mix(h, W=2, seed=53)
        snaps = {1: m.snap}
        h.h2tap_load_snapshot(e, h.hot_path_tables(m.snap), 1)
        steps = []
        for k in range(8):
            hot, upd, first = m.step(n_neworder=100, n_delivery=20)
            snaps[2 + k] = m.snap
            steps.append((hot, upd, first))
        seen, errors, stop = [], [], threading.Event()
        hi = m.clock + chgen.DAY_US

        def queries():
            try:
                while not stop.is_set():
                    rs = h.h2tap_run_queries(e, [(h.H2TAP_Q6, [Q6_D_LO, hi, 1, 100000], 0),
                                                 (h.H2TAP_Q1, [chgen.TS_2025], 0)])
                    seen.append((rs[0].epoch, rs[0].to_numpy(), rs[1].to_numpy()))
                    for r in rs:
                        r.free()
            except Exception as x:  # pragma: no cover
                errors.append(x)

        th = threading.Thread(target=queries)
        th.start()
        try:
            for k, (hot, upd, first) in enumerate(steps):
                h.h2tap_refresh(e, hot, upd, 2 + k, first_row=first, flags=h.H2TAP_LOAD_ASYNC)
        finally:
            h.h2tap_sync(e)
            import time
            time.sleep(0.2)
            stop.set()
            th.join()
        assert not errors
        assert len({ep for ep, _, _ in seen}) >= 2
        first = {}
        for ep, r6, r1 in seen:  # every result of one epoch is identical ...
            if ep in first:
                f6, f1 = first[ep]
                assert all(np.array_equal(r6[k], f6[k]) for k in f6)
                assert all(np.array_equal(r1[k], f1[k]) for k in f1)
            else:
                first[ep] = (r6, r1)
        for ep, (r6, r1) in first.items():  # ... and equals the oracle on that epoch's snapshot
            s = snaps[ep]
            w6 = oracle.q6(s, Q6_D_LO, hi, 1, 100000)
            assert int(r6["count_rows"][0]) == w6["count"]
            assert int(r6["revenue"][0]) == (w6["revenue"] or 0)
            w1 = oracle.q1(s, chgen.TS_2025)
            assert np.array_equal(r1["count_order"], w1["count_order"])
            assert np.array_equal(r1["sum_amount"], w1["sum_amount"])
    finally:
        h.h2tap_close(e)


def test_random_updates_i32_i64_columns(h):
    """Random row updates of ol_quantity (I32) and ol_amount / ol_delivery_d (I64), including
    rows in the ragged last page and NULL timestamps, over several epochs."""
    e = h.h2tap_open(0)
    try:
        t = chgen.generate(1, 3, seed=54)
        t.pop("item")
        h.h2tap_load_snapshot(e, h.hot_path_tables(t), 1)
        L = Loader(h, e)
        L.epoch = 1
        rng = np.random.default_rng(54)
        n = len(t["order_line"]["ol_o_id"])
        for k in range(5):
            upd = {}
            for col, lo, hi in (("ol_quantity", 0, 12), ("ol_amount", 1, 1_000_000),
                                ("ol_delivery_d", chgen.TS_1995, chgen.TS_2025)):
                m = int(rng.integers(1, 5000))
                rows = np.concatenate([[n - 1, n - 2, 0], 1 + rng.choice(n - 3, size=m, replace=False)])
                rows = rows.astype(np.uint32)  # distinct, incl. the ragged last page and row 0
                m = len(rows)
                vals = rng.integers(lo, hi, size=m).astype(t["order_line"][col].dtype)
                if col == "ol_delivery_d":
                    vals[rng.random(m) < 0.2] = chgen.NULL_TS
                upd[col] = (rows, vals)
            upd = {"order_line": upd}
            t = oracle.apply_updates(t, upd)
            L.epoch += 1
            h.h2tap_refresh(e, None, upd, L.epoch)
            check_epoch(L, t, chgen.TS_2025)
            cut = int(rng.integers(chgen.TS_1995, chgen.TS_2025))
            assert_q1(L.q(1, [cut]), oracle.q1(t, cut))
    finally:
        h.h2tap_close(e)


def test_key_column_updates_widen_zone_maps_and_detect_duplicates(h):
    e = h.h2tap_open(0)
    try:
        t = chgen.generate(1, 3, seed=55)
        t.pop("item")
        h.h2tap_load_snapshot(e, h.hot_path_tables(t), 1)
        L = Loader(h, e)
        # move some orders (and their lines) to fresh o_ids far outside the loaded key box
        o = t["orders"]
        sel = np.array([0, 5, 1000, len(o["o_id"]) - 1], np.uint32)
        new_ids = np.array([5_000_000, 5_000_001, 7_000_000, 9_999_999], np.int32)
        ol = t["order_line"]
        lines = [np.flatnonzero((ol["ol_w_id"] == o["o_w_id"][i]) & (ol["ol_d_id"] == o["o_d_id"][i])
                                & (ol["ol_o_id"] == o["o_id"][i])) for i in sel]
        ol_rows = np.concatenate(lines).astype(np.uint32)
        ol_vals = np.concatenate([np.full(len(x), v, np.int32) for x, v in zip(lines, new_ids)])
        upd = {"orders": {"o_id": (sel, new_ids)}, "order_line": {"ol_o_id": (ol_rows, ol_vals)}}
        t = oracle.apply_updates(t, upd)
        h.h2tap_refresh(e, None, upd, 2)
        L.epoch = 2
        want = oracle.q18(t, -1)
        assert_q18(L.q(18, [-1]), want)
        assert_q18(L.q(18, [-1], flags=4), want)
        assert set(new_ids.tolist()) <= set(want["o_id"].tolist())
        # a customer key updated onto another's -> duplicate build key
        upd = {"customer": {"c_id": (np.array([0], np.uint32), np.array([t["customer"]["c_id"][1]], np.int32))}}
        h.h2tap_refresh(e, None, upd, 3)
        with pytest.raises(h.H2tapError) as ei:
            h.h2tap_run_query(e, h.H2TAP_Q18)
        assert ei.value.status == h.H2TAP_EDUPKEY
    finally:
        h.h2tap_close(e)


def test_entry_and_amount_updates_keep_q18_order_exact(h):
    """Updates that move o_entry_d far below / above the loaded range and make amounts negative
    change the ORDER BY plan's field widths (carry records): element-wise parity
    at several HAVING thresholds, on every epoch."""
    e = h.h2tap_open(0)
    try:
        t = chgen.generate(1, 3, seed=57)
        t.pop("item")
        h.h2tap_load_snapshot(e, h.hot_path_tables(t), 1)
        L = Loader(h, e)
        o, ol = t["orders"], t["order_line"]
        rng = np.random.default_rng(57)
        sel = np.sort(rng.choice(len(o["o_id"]), 6, replace=False)).astype(np.uint32)
        ent = np.array([o["o_entry_d"].min() - 10 ** 12, o["o_entry_d"].max() + 10 ** 12, -5, 0,
                        o["o_entry_d"].max() + 1, 1], np.int64)
        lines = np.sort(rng.choice(len(ol["ol_o_id"]), 500, replace=False)).astype(np.uint32)
        amt = rng.integers(-10 ** 9, 10 ** 9, size=500).astype(np.int64)
        for k, upd in enumerate([{"orders": {"o_entry_d": (sel, ent)}},
                                 {"order_line": {"ol_amount": (lines, amt)}}]):
            t = oracle.apply_updates(t, upd)
            h.h2tap_refresh(e, None, upd, 2 + k)
            L.epoch = 2 + k
            for having in (Q18_HAVING, -1, -(10 ** 10), int(np.percentile(np.abs(amt), 50))):
                assert_q18(L.q(18, [having]), oracle.q18(t, having))
    finally:
        h.h2tap_close(e)


def test_update_errors(h):
    e = h.h2tap_open(0)
    try:
        t = chgen.generate(1, 2, seed=56)
        h.h2tap_load_snapshot(e, h.hot_path_tables(t), 1)
        n = len(t["order_line"]["ol_o_id"])
        ok = {"order_line": {"ol_quantity": (np.array([1], np.uint32), np.array([3], np.int32))}}
        cases = [
            ({"order_line": {"ol_quantity": (np.array([n], np.uint32), np.array([3], np.int32))}}, h.H2TAP_EINVAL),
            ({"orders": {"o_carrier_id": (np.array([0], np.uint32), np.array([3], np.int32))}}, h.H2TAP_EPLAN),
        ]
        for upd, status in cases:
            with pytest.raises(h.H2tapError) as ei:
                h.h2tap_refresh(e, None, upd, 2)
            assert ei.value.status == status
        with pytest.raises(ValueError):  # binding: dtype of the values must be the schema's
            h.h2tap_refresh(e, None, {"order_line": {"ol_quantity": (np.array([1], np.uint32),
                                                                     np.array([3], np.int64))}}, 2)
        h.h2tap_refresh(e, None, ok, 2)
        with pytest.raises(h.H2tapError) as ei:
            h.h2tap_refresh(e, None, ok, 2)
        assert ei.value.status == h.H2TAP_ESTALE
        # failed calls left the published snapshot intact
        assert h.h2tap_sync(e) == 2
        t2 = oracle.apply_updates(t, ok)
        L = Loader(h, e)
        assert_q6(L.q(6), oracle.q6(t2, Q6_D_LO, Q6_D_HI, Q6_Q_LO, Q6_Q_HI))
    finally:
        h.h2tap_close(e)


def test_full_size_w100_delivery_epoch(h):
    """BASELINE configs[1] size (W=100, 30M order_line rows): two epochs of NewOrder appends and
    Delivery updates (the second takes the page catch-up path), compared with the oracle."""
    e = h.h2tap_open(0)
    try:
        m = Mix(h, W=100, seed=1)
        h.h2tap_load_snapshot(e, h.hot_path_tables(m.snap), 1)
        for k in range(2):
            hot, upd, first = m.step(n_neworder=2000, n_delivery=1000)
            h.h2tap_refresh(e, hot, upd, 2 + k, first_row=first)
        L = Loader(h, e)
        check_epoch(L, m.snap, m.clock)
        st = h.h2tap_get_store_stats(e)
        assert st["cow_full_copies"] == 1 and st["cow_pages_copied"] > 0
    finally:
        h.h2tap_close(e)


def test_delivery_deletes_new_order_rows_q3(h):
    """Delivery's DELETE FROM new_order on the device store (R35): a tombstone update of
    new_order.no_deleted, copy-on-write like every update, published with the epoch's appends
    (NewOrder inserts orders, lines AND new_order rows). CH Q3 — the query that joins new_order —
    must equal the oracle on the visible snapshot (deleted rows removed; pinned to SQLite's
    DELETE in test_delivery_oracle.py) epoch after epoch, with no reload of new_order."""
    from chref import visible
    from test_oracle_q3 import Q3_LO
    W, seed = 2, 57
    plans = (h.H2TAP_Q3, h.H2TAP_Q18)
    snap = chgen.generate(1, W + 1, seed=seed)
    item = snap.pop("item")
    dl = chgen.DeliveryState()
    dl.add(snap["orders"], 0, 0, 0)
    no = chgen.NewOrderState(1, W + 1)
    e = h.h2tap_open(0)
    try:
        epoch = 1
        h.h2tap_load_snapshot(e, h.hot_path_tables(snap, plans), epoch)
        clock = chgen.TS_2025 + 5 * chgen.DAY_US
        lo = chgen.TS_1995
        deleted = 0
        for b in range(4):
            n_o, n_ol, n_no = (len(snap["orders"]["o_id"]), len(snap["order_line"]["ol_o_id"]),
                               len(snap["new_order"]["no_o_id"]))
            delta = chgen.neworder_batch(no, 200, seed=seed, batch=b, item=item)
            dl.add(delta["orders"], n_o, n_ol, n_no)
            w, carrier = chgen.delivery_inputs(30, seed=seed, batch=b, w_lo=1, w_hi=W + 1)
            upd = chgen.delivery_batch(dl, w, carrier, clock)
            clock += 31_000
            deleted += len(upd["new_order"]["no_deleted"][0])
            grown = {t: (_concat(snap[t], delta[t]) if t in delta else snap[t]) for t in snap}
            snap = oracle.apply_updates(grown, upd)
            epoch += 1
            dev = h.hot_path_tables({**delta, "customer": snap["customer"]}, plans)
            dev.pop("customer")
            dev_upd = {"new_order": upd["new_order"]}  # Q3/Q18 read no other updated column
            h.h2tap_refresh(e, dev, dev_upd, epoch, first_row={"orders": n_o, "order_line": n_ol, "new_order": n_no})
            for prefix in (b"A", b""):
                code = (prefix[0] << 8) if prefix else 0
                r = h.h2tap_run_query(e, h.H2TAP_Q3, [lo, code])
                got = r.to_numpy()
                r.free()
                want = oracle.q3(visible(snap), lo, prefix)
                for k in want:
                    assert np.array_equal(got[k], want[k]), (b, prefix, k)
            # the tombstones matter: with the deleted rows still there Q3 would differ
            assert len(oracle.q3(snap | {"new_order": {c: v for c, v in snap["new_order"].items()
                                                        if c != "no_deleted"}}, lo, b"")["ol_o_id"]) > \
                len(oracle.q3(visible(snap), lo, b"")["ol_o_id"])
        assert deleted > 0
        assert h.h2tap_get_store_stats(e)["rows_updated"] >= deleted
    finally:
        h.h2tap_close(e)
