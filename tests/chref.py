"""Test-side helpers that pin the oracle to things other than itself.

* ``sqlite_*``: load generated tables into stdlib ``sqlite3`` (NULL stored as SQL NULL,
  not as the sentinel) and run the literal CH-benCHmark SQL (SURVEY.md Appendix A.1
  [EXT]) with timestamp literals replaced by their int64-µs constants and money
  constants by cents (R4, R6).
* ``brute_*``: pure-Python nested loops over the cartesian product for tiny tables.
* ``golden``: the hand-derived fixture in tests/golden/.

None of this imports the product package or the oracle's C code.
"""
from __future__ import annotations

import datetime as dt
import itertools
import json
import os
import sqlite3

import numpy as np

NULL_SENTINEL = np.iinfo(np.int64).min
GOLDEN = os.path.join(os.path.dirname(os.path.abspath(__file__)), "golden")


def iso_us(s: str) -> int:
    t = dt.datetime.fromisoformat(s).replace(tzinfo=dt.timezone.utc)
    return (int(t.replace(microsecond=0).timestamp()) * 1_000_000) + t.microsecond


def ts_param(v) -> int:
    """A fixture parameter: an ISO timestamp string (-> int64 µs UTC) or a raw int64."""
    return iso_us(v) if isinstance(v, str) else int(v)


# CH-benCHmark literal constants, converted independently of the oracle and the library.
Q1_CUTOFF = iso_us("2007-01-02T00:00:00")
Q6_D_LO = iso_us("1999-01-01T00:00:00")
Q6_D_HI = iso_us("2020-01-01T00:00:00")
Q6_Q_LO, Q6_Q_HI = 1, 100000
Q18_HAVING = 200 * 100


# ------------------------------------------------------------------ SQLite --
def sqlite_load(tables):
    db = sqlite3.connect(":memory:")
    ol, o, c = tables["order_line"], tables["orders"], tables["customer"]
    db.execute("CREATE TABLE order_line (ol_w_id INT, ol_d_id INT, ol_o_id INT, ol_number INT,"
               " ol_delivery_d INT, ol_quantity INT, ol_amount INT, ol_i_id INT)")
    db.execute("CREATE TABLE orders (o_w_id INT, o_d_id INT, o_id INT, o_c_id INT, o_ol_cnt INT,"
               " o_entry_d INT, o_carrier_id INT)")
    db.execute("CREATE TABLE customer (c_w_id INT, c_d_id INT, c_id INT, c_last INT)")
    deliv = [None if int(v) == NULL_SENTINEL else int(v) for v in ol["ol_delivery_d"]]
    iid = ol["ol_i_id"].tolist() if "ol_i_id" in ol else [None] * len(deliv)
    db.executemany("INSERT INTO order_line VALUES (?,?,?,?,?,?,?,?)",
                   zip(ol["ol_w_id"].tolist(), ol["ol_d_id"].tolist(), ol["ol_o_id"].tolist(),
                       ol["ol_number"].tolist(), deliv, ol["ol_quantity"].tolist(),
                       ol["ol_amount"].tolist(), iid))
    carrier = [None if int(v) == -1 else int(v) for v in o["o_carrier_id"]]
    db.executemany("INSERT INTO orders VALUES (?,?,?,?,?,?,?)",
                   zip(o["o_w_id"].tolist(), o["o_d_id"].tolist(), o["o_id"].tolist(),
                       o["o_c_id"].tolist(), o["o_ol_cnt"].tolist(), o["o_entry_d"].tolist(),
                       carrier))
    db.executemany("INSERT INTO customer VALUES (?,?,?,?)",
                   zip(c["c_w_id"].tolist(), c["c_d_id"].tolist(), c["c_id"].tolist(),
                       c["c_last"].tolist()))
    db.execute("CREATE INDEX io ON orders (o_w_id, o_d_id, o_id)")
    db.execute("CREATE INDEX ic ON customer (c_w_id, c_d_id, c_id)")
    db.execute("CREATE INDEX il ON order_line (ol_w_id, ol_d_id, ol_o_id)")
    if "item" in tables and "i_data" in tables["item"]:
        it = tables["item"]
        db.execute("CREATE TABLE item (i_id INT, i_data TEXT)")
        db.executemany("INSERT INTO item VALUES (?,?)",
                       zip(it["i_id"].tolist(), [bytes(x).decode("latin-1") for x in it["i_data"]]))
        db.execute("CREATE INDEX ii ON item (i_id)")
    if "c_state" in c:
        db.execute("ALTER TABLE customer ADD COLUMN c_state TEXT")
        db.executemany("UPDATE customer SET c_state = ? WHERE rowid = ?",
                       [(bytes(x).decode("latin-1"), i + 1) for i, x in enumerate(c["c_state"])])
    if "new_order" in tables:
        no = live_new_order(tables["new_order"])
        db.execute("CREATE TABLE new_order (no_w_id INT, no_d_id INT, no_o_id INT)")
        db.executemany("INSERT INTO new_order VALUES (?,?,?)",
                       zip(no["no_w_id"].tolist(), no["no_d_id"].tolist(), no["no_o_id"].tolist()))
        db.execute("CREATE INDEX ino ON new_order (no_w_id, no_d_id, no_o_id)")
    db.execute("PRAGMA case_sensitive_like = ON")  # SQL LIKE is case-sensitive
    return db


def sqlite_q6(db, d_lo, d_hi, q_lo, q_hi):
    (rev,) = db.execute(
        "SELECT SUM(ol_amount) AS revenue FROM order_line "
        "WHERE ol_delivery_d >= ? AND ol_delivery_d < ? AND ol_quantity BETWEEN ? AND ?",
        (d_lo, d_hi, q_lo, q_hi)).fetchone()
    return rev


def sqlite_q1(db, cutoff):
    return db.execute(
        "SELECT ol_number, SUM(ol_quantity) AS sum_qty, SUM(ol_amount) AS sum_amount,"
        " AVG(ol_quantity) AS avg_qty, AVG(ol_amount) / 100.0 AS avg_amount, COUNT(*) AS count_order "
        "FROM order_line WHERE ol_delivery_d > ? GROUP BY ol_number ORDER BY ol_number",
        (cutoff,)).fetchall()


def sqlite_q18(db, having):
    return db.execute(
        "SELECT c_last, c_id, o_id, o_entry_d, o_ol_cnt, SUM(ol_amount) AS amount_sum, o_w_id, o_d_id "
        "FROM customer, orders, order_line "
        "WHERE c_id = o_c_id AND c_w_id = o_w_id AND c_d_id = o_d_id "
        "  AND ol_w_id = o_w_id AND ol_d_id = o_d_id AND ol_o_id = o_id "
        "GROUP BY o_id, o_w_id, o_d_id, c_id, c_last, o_entry_d, o_ol_cnt "
        "HAVING SUM(ol_amount) > ? ORDER BY amount_sum DESC, o_entry_d",
        (having,)).fetchall()


def sqlite_q14(db, d_lo, d_hi, prefix="PR"):
    """CH Q14 verbatim, money converted to currency units per row (ol_amount / 100.0)."""
    return db.execute(
        "SELECT 100.00 * SUM(CASE WHEN i_data LIKE ? THEN ol_amount / 100.0 ELSE 0 END)"
        " / (1 + SUM(ol_amount / 100.0)) AS promo_revenue,"
        " SUM(CASE WHEN i_data LIKE ? THEN ol_amount ELSE 0 END), SUM(ol_amount), COUNT(*) "
        "FROM order_line, item WHERE ol_i_id = i_id AND ol_delivery_d >= ? AND ol_delivery_d < ?",
        (prefix + "%", prefix + "%", d_lo, d_hi)).fetchone()


def sqlite_q12(db, d_hi):
    return db.execute(
        "SELECT o_ol_cnt,"
        " SUM(CASE WHEN o_carrier_id = 1 OR o_carrier_id = 2 THEN 1 ELSE 0 END) AS high_line_count,"
        " SUM(CASE WHEN o_carrier_id <> 1 AND o_carrier_id <> 2 THEN 1 ELSE 0 END) AS low_line_count "
        "FROM orders, order_line WHERE ol_w_id = o_w_id AND ol_d_id = o_d_id AND ol_o_id = o_id"
        " AND o_entry_d <= ol_delivery_d AND ol_delivery_d < ? GROUP BY o_ol_cnt ORDER BY o_ol_cnt",
        (d_hi,)).fetchall()


def sqlite_q4(db, e_lo, e_hi):
    return db.execute(
        "SELECT o_ol_cnt, COUNT(*) AS order_count FROM orders "
        "WHERE o_entry_d >= ? AND o_entry_d < ? AND EXISTS (SELECT * FROM order_line"
        " WHERE o_id = ol_o_id AND o_w_id = ol_w_id AND o_d_id = ol_d_id AND ol_delivery_d >= o_entry_d) "
        "GROUP BY o_ol_cnt ORDER BY o_ol_cnt", (e_lo, e_hi)).fetchall()


def sqlite_q3(db, entry_lo, prefix="A"):
    """CH Q3 verbatim (timestamp literal as int64 us)."""
    return db.execute(
        "SELECT ol_o_id, ol_w_id, ol_d_id, SUM(ol_amount) AS revenue, o_entry_d "
        "FROM customer, new_order, orders, order_line "
        "WHERE c_state LIKE ? AND c_id = o_c_id AND c_w_id = o_w_id AND c_d_id = o_d_id "
        "  AND no_w_id = o_w_id AND no_d_id = o_d_id AND no_o_id = o_id "
        "  AND ol_w_id = o_w_id AND ol_d_id = o_d_id AND ol_o_id = o_id AND o_entry_d > ? "
        "GROUP BY ol_o_id, ol_w_id, ol_d_id, o_entry_d ORDER BY revenue DESC, o_entry_d",
        (prefix + "%", entry_lo)).fetchall()


def sqlite_delivery(db, w, carrier, ts, districts):
    """One TPC-C Delivery transaction (TPC-C 2.7.4.2 [EXT]) as SQL: for each district, the
    oldest undelivered order (new_order = orders with a NULL carrier) gets the carrier and its
    lines get delivery date ts, and (when the database holds new_order) its new_order row is
    deleted."""
    has_no = db.execute("SELECT name FROM sqlite_master WHERE name = 'new_order'").fetchone() is not None
    for d in range(1, districts + 1):
        (o,) = db.execute("SELECT MIN(o_id) FROM orders WHERE o_w_id = ? AND o_d_id = ? "
                          "AND o_carrier_id IS NULL", (w, d)).fetchone()
        if o is None:
            continue
        if has_no:
            db.execute("DELETE FROM new_order WHERE no_w_id = ? AND no_d_id = ? AND no_o_id = ?", (w, d, o))
        db.execute("UPDATE orders SET o_carrier_id = ? WHERE o_w_id = ? AND o_d_id = ? AND o_id = ?",
                   (carrier, w, d, o))
        db.execute("UPDATE order_line SET ol_delivery_d = ? "
                   "WHERE ol_w_id = ? AND ol_d_id = ? AND ol_o_id = ?", (ts, w, d, o))


def live_new_order(no):
    """The new_order rows a query sees: those without a Delivery tombstone (no_deleted = 1 is the
    device store's record of DELETE FROM new_order, R35) — the plain definition of a
    deleted row, which simply is not there."""
    if "no_deleted" not in no:
        return no
    keep = np.asarray(no["no_deleted"]) == 0
    return {c: np.asarray(v)[keep] for c, v in no.items() if c != "no_deleted"}


def visible(tables):
    """A table set as SQL sees it: deleted new_order rows removed."""
    out = dict(tables)
    if "new_order" in out:
        out["new_order"] = live_new_order(out["new_order"])
    return out


def sqlite_column(db, table, column, null):
    """A column in insertion (rowid) order, SQL NULL mapped back to the sentinel ``null``."""
    return [null if v is None else v
            for (v,) in db.execute(f"SELECT {column} FROM {table} ORDER BY rowid")]


# -------------------------------------------------------------- brute force --
def _rows(t, cols):
    return list(zip(*[t[c].tolist() for c in cols]))


def _null(v):
    return None if v == NULL_SENTINEL else v


def brute_q6(tables, d_lo, d_hi, q_lo, q_hi):
    total, cnt = None, 0
    for (d, q, a) in _rows(tables["order_line"], ["ol_delivery_d", "ol_quantity", "ol_amount"]):
        d = _null(d)
        if d is None:
            continue
        if d_lo <= d < d_hi and q_lo <= q <= q_hi:
            total = a if total is None else total + a
            cnt += 1
    return total, cnt


def brute_q1(tables, cutoff):
    groups = {}
    for (n, d, q, a) in _rows(tables["order_line"],
                              ["ol_number", "ol_delivery_d", "ol_quantity", "ol_amount"]):
        d = _null(d)
        if d is not None and d > cutoff:
            g = groups.setdefault(n, [0, 0, 0])
            g[0] += q
            g[1] += a
            g[2] += 1
    return [(n, g[0], g[1], g[0] / g[2], g[1] / g[2] / 100.0, g[2]) for n, g in sorted(groups.items())]


def brute_q18(tables, having):
    """WHERE over the full cartesian product customer × orders × order_line."""
    C = _rows(tables["customer"], ["c_w_id", "c_d_id", "c_id", "c_last"])
    O = _rows(tables["orders"], ["o_w_id", "o_d_id", "o_id", "o_c_id", "o_ol_cnt", "o_entry_d"])
    L = _rows(tables["order_line"], ["ol_w_id", "ol_d_id", "ol_o_id", "ol_amount"])
    groups = {}
    for (cw, cd, cid, clast), (ow, od, oid, ocid, olcnt, oentry), (lw, ld, lo, la) in \
            itertools.product(C, O, L):
        if cid == ocid and cw == ow and cd == od and lw == ow and ld == od and lo == oid:
            k = (oid, ow, od, cid, clast, oentry, olcnt)
            groups[k] = groups.get(k, 0) + la
    out = [(k[4], k[3], k[0], k[5], k[6], s, k[1], k[2]) for k, s in groups.items() if s > having]
    out.sort(key=lambda r: (-r[5], r[3], r[6], r[7], r[2], r[1], r[0], r[4]))
    return out


def brute_q3(tables, entry_lo, prefix=b"A"):
    """CH Q3's WHERE over the cartesian product customer x new_order x orders x order_line,
    the conjunction evaluated in two stages (conjuncts without order_line first, over
    customer x new_order x orders; then the order_line conjuncts over that x order_line)."""
    C = list(zip(tables["customer"]["c_w_id"].tolist(), tables["customer"]["c_d_id"].tolist(),
                 tables["customer"]["c_id"].tolist(), [bytes(x) for x in tables["customer"]["c_state"]]))
    NO = _rows(tables["new_order"], ["no_w_id", "no_d_id", "no_o_id"])
    O = _rows(tables["orders"], ["o_w_id", "o_d_id", "o_id", "o_c_id", "o_entry_d"])
    L = _rows(tables["order_line"], ["ol_w_id", "ol_d_id", "ol_o_id", "ol_amount"])
    stage = [(ow, od, oid, oent)
             for (cw, cd, cid, cst), (nw, nd, no), (ow, od, oid, ocid, oent) in itertools.product(C, NO, O)
             if cst.startswith(prefix) and cid == ocid and cw == ow and cd == od
             and nw == ow and nd == od and no == oid and oent > entry_lo]
    groups = {}
    for (ow, od, oid, oent), (lw, ld, lo, la) in itertools.product(stage, L):
        if lw == ow and ld == od and lo == oid:
            k = (lo, lw, ld, oent)
            groups[k] = groups.get(k, 0) + la
    out = [(k[0], k[1], k[2], s, k[3]) for k, s in groups.items()]
    out.sort(key=lambda r: (-r[3], r[4], r[1], r[2], r[0]))
    return out


def brute_q14(tables, d_lo, d_hi, prefix=b"PR"):
    """(sum_promo, sum_amount, count) over the cartesian product order_line × item."""
    L = _rows(tables["order_line"], ["ol_i_id", "ol_delivery_d", "ol_amount"])
    items = list(zip(tables["item"]["i_id"].tolist(), [bytes(x) for x in tables["item"]["i_data"]]))
    sp = sa = cnt = 0
    for (iid, d, a), (i_id, data) in itertools.product(L, items):
        d = _null(d)
        if iid == i_id and d is not None and d_lo <= d < d_hi:
            sp += a if data.startswith(prefix) else 0
            sa += a
            cnt += 1
    return sp, sa, cnt


def brute_q12(tables, d_hi):
    O = _rows(tables["orders"], ["o_w_id", "o_d_id", "o_id", "o_ol_cnt", "o_carrier_id", "o_entry_d"])
    L = _rows(tables["order_line"], ["ol_w_id", "ol_d_id", "ol_o_id", "ol_delivery_d"])
    groups = {}
    for (ow, od, oid, cnt, car, ent), (lw, ld, lo, d) in itertools.product(O, L):
        d = _null(d)
        if lw == ow and ld == od and lo == oid and d is not None and ent <= d and d < d_hi:
            g = groups.setdefault(cnt, [0, 0])
            if car != -1 and car in (1, 2):
                g[0] += 1
            if car != -1 and car not in (1, 2):
                g[1] += 1
    return [(k, g[0], g[1]) for k, g in sorted(groups.items())]


def brute_q4(tables, e_lo, e_hi):
    O = _rows(tables["orders"], ["o_w_id", "o_d_id", "o_id", "o_ol_cnt", "o_entry_d"])
    L = _rows(tables["order_line"], ["ol_w_id", "ol_d_id", "ol_o_id", "ol_delivery_d"])
    groups = {}
    for (ow, od, oid, cnt, ent) in O:
        if not (e_lo <= ent < e_hi):
            continue
        if any(lw == ow and ld == od and lo == oid and _null(d) is not None and d >= ent
               for (lw, ld, lo, d) in L):
            groups[cnt] = groups.get(cnt, 0) + 1
    return sorted(groups.items())


# ------------------------------------------------------------------- golden --
def golden(name="tiny_ch.json"):
    with open(os.path.join(GOLDEN, name)) as f:
        g = json.load(f)
    conv = {"ol_delivery_d": True, "o_entry_d": True}
    tables = {}
    for t in ("order_line", "orders", "customer"):
        cols = g[t]["columns"]
        rows = g[t]["rows"]
        tab = {}
        for j, c in enumerate(cols):
            vals = [r[j] for r in rows]
            if c in conv:
                tab[c] = np.array([NULL_SENTINEL if v is None else iso_us(v) for v in vals], np.int64)
            elif c in ("ol_amount",):
                tab[c] = np.array(vals, np.int64)
            else:
                tab[c] = np.array(vals, np.int32)
        tables[t] = tab
    ol = tables["order_line"]
    n = len(ol["ol_w_id"])
    ol.setdefault("ol_i_id", np.ones(n, np.int32))
    ol.setdefault("ol_supply_w_id", ol["ol_w_id"].copy())
    o = tables["orders"]
    m = len(o["o_w_id"])
    o.setdefault("o_carrier_id", np.full(m, -1, np.int32))
    o.setdefault("o_all_local", np.ones(m, np.int32))
    return tables, g["expected"]


def table_rows(tables, t):
    return len(next(iter(tables[t].values())))


def canon_rows(cols: dict, names):
    """Rows as a sorted list of tuples (canonical full-row sort for set comparison)."""
    return sorted(zip(*[np.asarray(cols[n]).tolist() for n in names]))


def golden_next2(name="ch_next2.json"):
    """The NEXT-2 fixture as generator-shaped tables (+ params and expected values)."""
    with open(os.path.join(GOLDEN, name)) as f:
        g = json.load(f)
    ts_cols = ("ol_delivery_d", "o_entry_d")
    i64_cols = ("ol_amount",)
    tables = {}
    for t in ("orders", "order_line"):
        cols, rows = g[t]["columns"], g[t]["rows"]
        tab = {}
        for j, c in enumerate(cols):
            vals = [r[j] for r in rows]
            if c in ts_cols:
                tab[c] = np.array([NULL_SENTINEL if v is None else iso_us(v) for v in vals], np.int64)
            elif c in i64_cols:
                tab[c] = np.array(vals, np.int64)
            else:
                tab[c] = np.array(vals, np.int32)
        tables[t] = tab
    ol = tables["order_line"]
    n = len(ol["ol_w_id"])
    ol["ol_number"] = ol.get("ol_number", np.ones(n, np.int32))
    ol["ol_quantity"] = np.ones(n, np.int32)
    ol["ol_supply_w_id"] = ol["ol_w_id"].copy()
    o = tables["orders"]
    o["o_all_local"] = np.ones(len(o["o_id"]), np.int32)
    items = g["item"]["rows"]
    data = np.array([s.encode() for _, s in items], dtype="S50")
    b = np.frombuffer(data.tobytes(), np.uint8).reshape(-1, 50)
    tables["item"] = {"i_id": np.array([i for i, _ in items], np.int32),
                      "i_price": np.full(len(items), 100, np.int64), "i_data": data,
                      "i_data_p2": ((b[:, 0].astype(np.int32) << 8) | b[:, 1]).astype(np.int32)}
    tables["customer"] = {"c_w_id": np.zeros(0, np.int32), "c_d_id": np.zeros(0, np.int32),
                          "c_id": np.zeros(0, np.int32), "c_last": np.zeros(0, np.int32)}
    p = g["params"]
    params = {"q14": (iso_us(p["q14"][0]), iso_us(p["q14"][1]), p["q14"][2].encode()),
              "q12": (iso_us(p["q12"][0]),), "q4": (iso_us(p["q4"][0]), iso_us(p["q4"][1]))}
    return tables, params, g["expected"]


def golden_q3(name="ch_q3.json"):
    """The CH Q3 fixture as generator-shaped tables (+ params and expected rows)."""
    with open(os.path.join(GOLDEN, name)) as f:
        g = json.load(f)
    tables = {}
    for t in ("customer", "orders", "new_order", "order_line"):
        cols, rows = g[t]["columns"], g[t]["rows"]
        tab = {}
        for j, c in enumerate(cols):
            vals = [r[j] for r in rows]
            if c == "o_entry_d":
                tab[c] = np.array([iso_us(v) for v in vals], np.int64)
            elif c == "ol_amount":
                tab[c] = np.array(vals, np.int64)
            elif c == "c_state":
                tab[c] = np.array([v.encode() for v in vals], dtype="S2")
            else:
                tab[c] = np.array(vals, np.int32)
        tables[t] = tab
    c = tables["customer"]
    b = np.frombuffer(c["c_state"].tobytes(), np.uint8).reshape(-1, 2)
    c["c_state_p2"] = ((b[:, 0].astype(np.int32) << 8) | b[:, 1]).astype(np.int32)
    ol = tables["order_line"]
    n = len(ol["ol_w_id"])
    ol["ol_delivery_d"] = np.full(n, NULL_SENTINEL, np.int64)
    ol["ol_quantity"] = np.ones(n, np.int32)
    ol["ol_i_id"] = np.ones(n, np.int32)
    ol["ol_supply_w_id"] = ol["ol_w_id"].copy()
    tables["orders"]["o_all_local"] = np.ones(len(tables["orders"]["o_id"]), np.int32)
    p = g["params"]["q3"]
    want = [(r[0], r[1], r[2], r[3], iso_us(r[4])) for r in g["expected"]["q3"]]
    return tables, (iso_us(p[0]), p[1].encode()), want
