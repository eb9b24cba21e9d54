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
               " ol_delivery_d INT, ol_quantity INT, ol_amount INT)")
    db.execute("CREATE TABLE orders (o_w_id INT, o_d_id INT, o_id INT, o_c_id INT, o_ol_cnt INT,"
               " o_entry_d INT, o_carrier_id INT)")
    db.execute("CREATE TABLE customer (c_w_id INT, c_d_id INT, c_id INT, c_last INT)")
    deliv = [None if int(v) == NULL_SENTINEL else int(v) for v in ol["ol_delivery_d"]]
    db.executemany("INSERT INTO order_line VALUES (?,?,?,?,?,?,?)",
                   zip(ol["ol_w_id"].tolist(), ol["ol_d_id"].tolist(), ol["ol_o_id"].tolist(),
                       ol["ol_number"].tolist(), deliv, ol["ol_quantity"].tolist(),
                       ol["ol_amount"].tolist()))
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


def sqlite_delivery(db, w, carrier, ts, districts):
    """One TPC-C Delivery transaction (TPC-C 2.7.4.2 [EXT]) as SQL: for each district, the
    oldest undelivered order (new_order = orders with a NULL carrier) gets the carrier and its
    lines get delivery date ts."""
    for d in range(1, districts + 1):
        (o,) = db.execute("SELECT MIN(o_id) FROM orders WHERE o_w_id = ? AND o_d_id = ? "
                          "AND o_carrier_id IS NULL", (w, d)).fetchone()
        if o is None:
            continue
        db.execute("UPDATE orders SET o_carrier_id = ? WHERE o_w_id = ? AND o_d_id = ? AND o_id = ?",
                   (carrier, w, d, o))
        db.execute("UPDATE order_line SET ol_delivery_d = ? "
                   "WHERE ol_w_id = ? AND ol_d_id = ? AND ol_o_id = ?", (ts, w, d, o))


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
