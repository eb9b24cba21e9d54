"""chgen — seeded synthetic CH-benCHmark / TPC-C table generator.

This module is INPUT ONLY: it produces the column arrays that both the CPU
oracle (``oracle/``) and the CUDA path (``paper_conf_cidr_appuswamykpa17_b200``)
consume. It contains none of the queries' arithmetic (no filter, join,
aggregate or sort of the CH queries) — the two sides share nothing else.

Population follows TPC-C §4.3.3.1 as restated in SURVEY.md Appendix A.3
([EXT]: the paper itself, PAPER.md, evaluates TPC-H Q6 on lineitem, L687-688,
and never defines the CH tables). Two modes (reading R9 / SURVEY B9):

* ``strict`` — TPC-C population: delivered lines (o_id < 2101) carry
  delivery_d = o_entry_d = LOAD_TS, quantity 5, amount 0.00; undelivered lines
  have delivery NULL and amount U[0.01, 9999.99].
* ``spread`` — the default for parity and perf: o_entry_d uniform in
  [1995-01-01, 2025-01-01), delivery_d = o_entry_d + U[0, 30 d) for delivered
  lines, quantity U[1, 10], amount U[0.01, 9999.99] for every line.

Encodings (R4-R6): ids int32; timestamps int64 µs
since 1970-01-01 UTC with SQL NULL stored as INT64_MIN; money int64 cents;
o_carrier_id NULL stored as -1; c_last an int32 dictionary code 0..999; i_data the
TPC-C string (bytes) plus ``i_data_p2`` = (byte0 << 8) | byte1, the device encoding of its
first two characters (what CH Q14's ``LIKE 'PR%'`` needs; R29).

Every warehouse w draws from its own stream ``Philox(key=[seed, w])`` (item
uses w = 0), so any warehouse range [a, b) reproduces byte-identical rows to
the same slice of a full generation — the basis of sharding across ranks.
"""
from __future__ import annotations

import datetime as _dt
from collections import deque
from dataclasses import dataclass, field

import numpy as np

__all__ = [
    "Scale", "TINY", "FULL", "NULL_TS", "LOAD_TS", "TS_1995", "TS_2025",
    "DAY_US", "ts_us", "generate", "generate_item", "neworder_delta",
    "warehouse_ranges", "concat_tables", "TABLE_COLUMNS", "NewOrderState", "neworder_batch",
    "ROW_DTYPES", "to_records", "DeliveryState", "delivery_inputs", "delivery_batch",
    "i_data_prefix2", "prefix2", "layout_matrix", "encode_layout",
]


def ts_us(iso: str) -> int:
    """int64 µs since the Unix epoch (UTC) of an ISO date/time string."""
    t = _dt.datetime.fromisoformat(iso).replace(tzinfo=_dt.timezone.utc)
    return int(t.timestamp()) * 1_000_000


NULL_TS = np.iinfo(np.int64).min          # SQL NULL for ol_delivery_d
LOAD_TS = ts_us("2015-01-01")             # strict-mode o_entry_d
TS_1995 = ts_us("1995-01-01")
TS_2025 = ts_us("2025-01-01")
DAY_US = 86_400 * 1_000_000
NURAND_C_LAST = 157                       # TPC-C run-time constant C for NURand(255,0,999)

# Column order of each table as the generator emits it (SoA, one ndarray each).
TABLE_COLUMNS = {
    "order_line": [("ol_w_id", np.int32), ("ol_d_id", np.int32), ("ol_o_id", np.int32),
                   ("ol_number", np.int32), ("ol_i_id", np.int32), ("ol_supply_w_id", np.int32),
                   ("ol_delivery_d", np.int64), ("ol_quantity", np.int32), ("ol_amount", np.int64)],
    "orders": [("o_w_id", np.int32), ("o_d_id", np.int32), ("o_id", np.int32),
               ("o_c_id", np.int32), ("o_ol_cnt", np.int32), ("o_carrier_id", np.int32),
               ("o_all_local", np.int32), ("o_entry_d", np.int64)],
    "customer": [("c_w_id", np.int32), ("c_d_id", np.int32), ("c_id", np.int32),
                 ("c_last", np.int32), ("c_state", "S2"), ("c_state_p2", np.int32)],
    # no_deleted: 1 once a Delivery has deleted the row (TPC-C 2.7.4.2 DELETE FROM new_order), kept
    # as an in-place update of a tombstone column so the device store stays append + update only
    # (R35); every generated / inserted row has 0
    "new_order": [("no_w_id", np.int32), ("no_d_id", np.int32), ("no_o_id", np.int32),
                  ("no_deleted", np.int32)],
    "item": [("i_id", np.int32), ("i_price", np.int64), ("i_data", "S50"), ("i_data_p2", np.int32)],
}


@dataclass(frozen=True)
class Scale:
    """Per-warehouse cardinalities. FULL is TPC-C; TINY is for brute force."""
    districts: int = 10
    orders_per_district: int = 3000
    customers_per_district: int = 3000
    items: int = 100_000
    min_ol_cnt: int = 5
    max_ol_cnt: int = 15

    @property
    def delivered_below(self) -> int:
        """o_id threshold for delivered orders: 2101 at 3000 orders (TPC-C)."""
        return self.orders_per_district * 7 // 10 + 1


FULL = Scale()
TINY = Scale(districts=2, orders_per_district=20, customers_per_district=20, items=100)


def _rng(seed: int, w: int) -> np.random.Generator:
    return np.random.Generator(np.random.Philox(key=np.array([seed, w], dtype=np.uint64)))


def _warehouse(w: int, seed: int, mode: str, sc: Scale):
    if mode not in ("strict", "spread"):
        raise ValueError(f"mode must be 'strict' or 'spread', not {mode!r}")
    if sc.orders_per_district > sc.customers_per_district:
        raise ValueError("o_c_id is a permutation of customers: need orders <= customers")
    rng = _rng(seed, w)
    D, O, C = sc.districts, sc.orders_per_district, sc.customers_per_district
    n_o = D * O

    # ---- orders (PK order: d, o_id) ------------------------------------
    o_d = np.repeat(np.arange(1, D + 1, dtype=np.int32), O)
    o_id = np.tile(np.arange(1, O + 1, dtype=np.int32), D)
    perm = rng.permuted(np.tile(np.arange(1, C + 1, dtype=np.int32), (D, 1)), axis=1)
    o_c_id = np.ascontiguousarray(perm[:, :O]).reshape(-1)
    o_ol_cnt = rng.integers(sc.min_ol_cnt, sc.max_ol_cnt + 1, size=n_o, dtype=np.int32)
    carrier = rng.integers(1, 11, size=n_o, dtype=np.int32)
    delivered = o_id < sc.delivered_below
    o_carrier = np.where(delivered, carrier, np.int32(-1)).astype(np.int32)
    if mode == "strict":
        o_entry = np.full(n_o, LOAD_TS, dtype=np.int64)
    else:
        o_entry = rng.integers(TS_1995, TS_2025, size=n_o, dtype=np.int64)

    # ---- order_line (PK order: d, o_id, ol_number) ----------------------
    n_ol = int(o_ol_cnt.sum())
    starts = np.zeros(n_o, dtype=np.int64)
    np.cumsum(o_ol_cnt[:-1], out=starts[1:])
    ol_o = np.repeat(o_id, o_ol_cnt)
    ol_d = np.repeat(o_d, o_ol_cnt)
    ol_number = (np.arange(n_ol, dtype=np.int64) - np.repeat(starts, o_ol_cnt) + 1).astype(np.int32)
    ol_i_id = rng.integers(1, sc.items + 1, size=n_ol, dtype=np.int32)
    ol_deliv_mask = np.repeat(delivered, o_ol_cnt)
    ol_entry = np.repeat(o_entry, o_ol_cnt)
    if mode == "strict":
        ol_delivery = np.where(ol_deliv_mask, ol_entry, NULL_TS)
        ol_qty = np.full(n_ol, 5, dtype=np.int32)
        amt = rng.integers(1, 1_000_000, size=n_ol, dtype=np.int64)
        ol_amount = np.where(ol_deliv_mask, np.int64(0), amt)
    else:
        lag = rng.integers(0, 30 * DAY_US, size=n_ol, dtype=np.int64)
        ol_delivery = np.where(ol_deliv_mask, ol_entry + lag, NULL_TS)
        ol_qty = rng.integers(1, 11, size=n_ol, dtype=np.int32)
        ol_amount = rng.integers(1, 1_000_000, size=n_ol, dtype=np.int64)

    # ---- customer (PK order: d, c_id) -----------------------------------
    c_d = np.repeat(np.arange(1, D + 1, dtype=np.int32), C)
    c_id = np.tile(np.arange(1, C + 1, dtype=np.int32), D)
    a = rng.integers(0, 256, size=D * C, dtype=np.int32)
    b = rng.integers(0, 1000, size=D * C, dtype=np.int32)
    nurand = ((a | b) + NURAND_C_LAST) % 1000
    c_last = np.where(c_id <= 1000, c_id - 1, nurand).astype(np.int32)
    # c_state: random a-string of 2 characters (TPC-C 4.3.3.1 [EXT]) over the same alphabet as
    # i_data; drawn LAST from the warehouse stream so that every earlier column is unchanged
    st = ALNUM[rng.integers(0, len(ALNUM), size=(D * C, 2))]
    c_state = np.ascontiguousarray(st).view("S2").reshape(D * C)

    wi = np.int32(w)
    ol = {
        "ol_w_id": np.full(n_ol, wi, dtype=np.int32), "ol_d_id": ol_d, "ol_o_id": ol_o,
        "ol_number": ol_number, "ol_i_id": ol_i_id,
        "ol_supply_w_id": np.full(n_ol, wi, dtype=np.int32),
        "ol_delivery_d": ol_delivery.astype(np.int64), "ol_quantity": ol_qty.astype(np.int32),
        "ol_amount": ol_amount.astype(np.int64),
    }
    orders = {
        "o_w_id": np.full(n_o, wi, dtype=np.int32), "o_d_id": o_d, "o_id": o_id,
        "o_c_id": o_c_id, "o_ol_cnt": o_ol_cnt, "o_carrier_id": o_carrier,
        "o_all_local": np.ones(n_o, dtype=np.int32), "o_entry_d": o_entry,
    }
    customer = {"c_w_id": np.full(D * C, wi, dtype=np.int32), "c_d_id": c_d, "c_id": c_id,
                "c_last": c_last, "c_state": c_state, "c_state_p2": prefix2(c_state)}
    # new_order: one row per undelivered order (TPC-C 4.3.3.1: the last 900 orders of each
    # district, NO_O_ID 2101..3000), in (d, o_id) order
    und = o_carrier == -1
    new_order = {"no_w_id": np.full(int(und.sum()), wi, dtype=np.int32), "no_d_id": o_d[und],
                 "no_o_id": o_id[und], "no_deleted": np.zeros(int(und.sum()), dtype=np.int32)}
    return {"order_line": ol, "orders": orders, "customer": customer, "new_order": new_order}


ALNUM = np.frombuffer(b"abcdefghijklmnopqrstuvwxyzABCDEFGHIJKLMNOPQRSTUVWXYZ0123456789", np.uint8)


def prefix2(strings) -> np.ndarray:
    """(byte0 << 8) | byte1 of each fixed-width byte string (0 for a missing byte): the device
    encoding of a string column's first two characters (R29)."""
    a = np.asarray(strings)
    width = max(a.dtype.itemsize, 2)
    b = np.frombuffer(a.astype(f"S{width}").tobytes(), np.uint8).reshape(-1, width)
    return ((b[:, 0].astype(np.int32) << 8) | b[:, 1].astype(np.int32)).astype(np.int32)


def i_data_prefix2(i_data) -> np.ndarray:
    """(byte0 << 8) | byte1 of each i_data string (0 for a missing byte)."""
    return prefix2(np.asarray(i_data, dtype="S50"))


def generate_item(seed: int = 1, scale: Scale = FULL):
    """item table (replicated on every rank), stream key [seed, 0]. i_data per TPC-C 4.3.3.1
    [EXT]: random a-string of length U[26, 50] over [a-zA-Z0-9]; 10 % contain "ORIGINAL" at a
    random position."""
    rng = _rng(seed, 0)
    n = scale.items
    price = rng.integers(100, 10_001, size=n, dtype=np.int64)
    length = rng.integers(26, 51, size=n)
    chars = ALNUM[rng.integers(0, len(ALNUM), size=(n, 50))]
    orig = rng.random(n) < 0.10
    pos = rng.integers(0, length - 8 + 1)
    for i in np.flatnonzero(orig):
        chars[i, pos[i]:pos[i] + 8] = np.frombuffer(b"ORIGINAL", np.uint8)
    chars[np.arange(50)[None, :] >= length[:, None]] = 0
    i_data = chars.view("S50").reshape(n)
    return {"i_id": np.arange(1, n + 1, dtype=np.int32), "i_price": price,
            "i_data": i_data, "i_data_p2": i_data_prefix2(i_data)}


def concat_tables(parts):
    """Concatenate a list of {table: {col: array}} dicts table by table."""
    out = {}
    for t in parts[0]:
        out[t] = {c: np.concatenate([p[t][c] for p in parts]) for c in parts[0][t]}
    return out


def generate(w_lo: int, w_hi: int | None = None, *, seed: int = 1, mode: str = "spread",
             scale: Scale = FULL, with_item: bool = True):
    """Tables for warehouses [w_lo, w_hi) (1-based ids). ``generate(1, W+1)`` is W warehouses.

    Returns ``{"order_line": {...}, "orders": {...}, "customer": {...}, "item": {...}}``
    with each column a contiguous numpy array in the dtype of TABLE_COLUMNS.
    """
    if w_hi is None:
        w_lo, w_hi = 1, w_lo + 1
    if not (1 <= w_lo <= w_hi):
        raise ValueError("warehouse ids are 1-based and w_lo <= w_hi")
    if w_hi == w_lo:
        empty = {t: {c: np.zeros(0, dtype=dt) for c, dt in cols}
                 for t, cols in TABLE_COLUMNS.items() if t != "item"}
        parts = [empty]
    else:
        parts = [_warehouse(w, seed, mode, scale) for w in range(w_lo, w_hi)]
    out = concat_tables(parts) if len(parts) > 1 else parts[0]
    if with_item:
        out["item"] = generate_item(seed, scale)
    return out


def warehouse_ranges(n_warehouses: int, world: int):
    """Contiguous warehouse ranges [lo, hi) per rank (R15)."""
    base, extra = divmod(n_warehouses, world)
    out, lo = [], 1
    for r in range(world):
        hi = lo + base + (1 if r < extra else 0)
        out.append((lo, hi))
        lo = hi
    return out


@dataclass
class NewOrderState:
    """Per-district next o_id for appended NewOrder transactions (config C5 input)."""
    w_lo: int
    w_hi: int
    scale: Scale = FULL
    next_o_id: dict = field(default_factory=dict)
    clock: int = TS_2025


def neworder_delta(state: NewOrderState, n_txn: int, *, seed: int, batch: int,
                   item=None):
    """Rows appended by ``n_txn`` TPC-C NewOrder transactions.

    Simplified TPC-C 2.4.1 input generation: district uniform, customer uniform,
    ol_cnt U[5,15], item uniform, qty U[1,10], amount = qty * i_price, delivery NULL,
    o_entry_d a logical clock starting 2025-01-01. No rollbacks in this delta.
    Returns ``{"order_line": {...}, "orders": {...}}`` for the appended rows only.
    """
    sc = state.scale
    rng = np.random.Generator(np.random.Philox(key=np.array([seed, 1 << 40 | batch], dtype=np.uint64)))
    if item is None:
        item = generate_item(seed, sc)
    cols_o = {c: [] for c, _ in TABLE_COLUMNS["orders"]}
    cols_l = {c: [] for c, _ in TABLE_COLUMNS["order_line"]}
    for _ in range(n_txn):
        w = int(rng.integers(state.w_lo, state.w_hi))
        d = int(rng.integers(1, sc.districts + 1))
        key = (w, d)
        o = state.next_o_id.get(key, sc.orders_per_district + 1)
        state.next_o_id[key] = o + 1
        c = int(rng.integers(1, sc.customers_per_district + 1))
        cnt = int(rng.integers(sc.min_ol_cnt, sc.max_ol_cnt + 1))
        state.clock += 1_000
        for k, v in (("o_w_id", w), ("o_d_id", d), ("o_id", o), ("o_c_id", c),
                     ("o_ol_cnt", cnt), ("o_carrier_id", -1), ("o_all_local", 1),
                     ("o_entry_d", state.clock)):
            cols_o[k].append(v)
        iids = rng.integers(1, sc.items + 1, size=cnt)
        qtys = rng.integers(1, 11, size=cnt)
        for n in range(cnt):
            i = int(iids[n])
            q = int(qtys[n])
            for k, v in (("ol_w_id", w), ("ol_d_id", d), ("ol_o_id", o), ("ol_number", n + 1),
                         ("ol_i_id", i), ("ol_supply_w_id", w), ("ol_delivery_d", int(NULL_TS)),
                         ("ol_quantity", q), ("ol_amount", q * int(item["i_price"][i - 1]))):
                cols_l[k].append(v)
    dts = {c: dt for t in ("orders", "order_line") for c, dt in TABLE_COLUMNS[t]}
    orders = {k: np.asarray(v, dtype=dts[k]) for k, v in cols_o.items()}
    return {"orders": orders,
            "order_line": {k: np.asarray(v, dtype=dts[k]) for k, v in cols_l.items()},
            "new_order": _new_order_rows(orders)}


def _new_order_rows(orders: dict) -> dict:
    """The new_order rows a NewOrder transaction inserts: one per new order (TPC-C 2.4.2.2)."""
    return {"no_w_id": orders["o_w_id"].astype(np.int32), "no_d_id": orders["o_d_id"].astype(np.int32),
            "no_o_id": orders["o_id"].astype(np.int32), "no_deleted": np.zeros(len(orders["o_id"]), np.int32)}


def neworder_batch(state: NewOrderState, n_txn: int, *, seed: int, batch: int, item=None):
    """Vectorised ``neworder_delta``: the rows appended by ``n_txn`` NewOrder transactions
    (district and customer uniform, ol_cnt U[5,15], item uniform, qty U[1,10],
    amount = qty * i_price, delivery NULL, o_id = next id of the district, o_entry_d a logical
    clock). Same semantics as ``neworder_delta``; used to drive config C5 at high rates."""
    sc = state.scale
    rng = np.random.Generator(np.random.Philox(key=np.array([seed, 1 << 41 | batch], dtype=np.uint64)))
    if item is None:
        item = generate_item(seed, sc)
    w = rng.integers(state.w_lo, state.w_hi, size=n_txn).astype(np.int32)
    d = rng.integers(1, sc.districts + 1, size=n_txn).astype(np.int32)
    c = rng.integers(1, sc.customers_per_district + 1, size=n_txn).astype(np.int32)
    cnt = rng.integers(sc.min_ol_cnt, sc.max_ol_cnt + 1, size=n_txn).astype(np.int32)
    # o_id: next id per (w, d), in transaction order
    key = w.astype(np.int64) * 64 + d
    order = np.argsort(key, kind="stable")
    ks = key[order]
    first = np.r_[True, ks[1:] != ks[:-1]]
    grp_start = np.maximum.accumulate(np.where(first, np.arange(n_txn), 0))
    rank_in_grp = np.arange(n_txn) - grp_start
    base = np.array([state.next_o_id.get((int(k) // 64, int(k) % 64), sc.orders_per_district + 1)
                     for k in ks[first]], dtype=np.int64)
    gid = np.cumsum(first) - 1
    o_sorted = base[gid] + rank_in_grp
    o_id = np.empty(n_txn, np.int64)
    o_id[order] = o_sorted
    for k, b, g in zip(ks[first], base, np.bincount(gid)):
        state.next_o_id[(int(k) // 64, int(k) % 64)] = int(b + g)
    entry = state.clock + 1_000 * np.arange(1, n_txn + 1, dtype=np.int64)
    state.clock = int(entry[-1]) if n_txn else state.clock
    n_ol = int(cnt.sum())
    starts = np.zeros(n_txn, np.int64)
    np.cumsum(cnt[:-1], out=starts[1:])
    number = (np.arange(n_ol) - np.repeat(starts, cnt) + 1).astype(np.int32)
    iid = rng.integers(1, sc.items + 1, size=n_ol).astype(np.int32)
    qty = rng.integers(1, 11, size=n_ol).astype(np.int32)
    amount = qty.astype(np.int64) * item["i_price"][iid - 1]
    orders = {"o_w_id": w, "o_d_id": d, "o_id": o_id.astype(np.int32), "o_c_id": c, "o_ol_cnt": cnt,
              "o_carrier_id": np.full(n_txn, -1, np.int32), "o_all_local": np.ones(n_txn, np.int32),
              "o_entry_d": entry}
    ol = {"ol_w_id": np.repeat(w, cnt), "ol_d_id": np.repeat(d, cnt),
          "ol_o_id": np.repeat(o_id.astype(np.int32), cnt), "ol_number": number, "ol_i_id": iid,
          "ol_supply_w_id": np.repeat(w, cnt), "ol_delivery_d": np.full(n_ol, NULL_TS, np.int64),
          "ol_quantity": qty, "ol_amount": amount}
    return {"orders": orders, "order_line": ol, "new_order": _new_order_rows(orders)}


# NSM record layouts of the host row store (one record per row, fields in schema order)
ROW_DTYPES = {t: np.dtype([(c, dt) for c, dt in cols]) for t, cols in TABLE_COLUMNS.items()}


def to_records(table: str, cols: dict) -> np.ndarray:
    """Columns -> NSM records (numpy structured array) of ``table``'s row layout."""
    n = len(next(iter(cols.values())))
    rec = np.empty(n, ROW_DTYPES[table])
    for c in ROW_DTYPES[table].names:
        rec[c] = cols[c]
    return rec


# ------------------------------------------------------------------ Delivery --
@dataclass
class DeliveryState:
    """The OLTP side's new_order table: per district (w, d), a FIFO of the undelivered orders in
    o_id order, each as (o_id, orders row, first order_line row, ol_cnt) — row positions in the
    host row store, which is what an in-place update names (NEXT-1).

    ``add(orders, o_row0, ol_row0, no_row0)`` registers a block of orders stored at orders rows
    ``o_row0 + i`` whose lines are stored contiguously, in the same order, from order_line row
    ``ol_row0`` on (true for ``generate`` tables and for ``neworder_batch`` deltas); with
    ``no_row0``, the k-th undelivered order of the block is new_order row ``no_row0 + k`` (true for
    both as well: their new_order rows list the undelivered orders in orders-row order), which a
    Delivery then deletes (a tombstone update of ``no_deleted``)."""
    districts: int = FULL.districts
    queues: dict = field(default_factory=dict)

    def add(self, orders: dict, o_row0: int = 0, ol_row0: int = 0, no_row0: int | None = None):
        cnt = orders["o_ol_cnt"].astype(np.int64)
        ol_first = ol_row0 + np.concatenate([[0], np.cumsum(cnt)[:-1]]) if len(cnt) else cnt
        pending = np.flatnonzero(orders["o_carrier_id"] == -1)
        w, d, o = orders["o_w_id"], orders["o_d_id"], orders["o_id"]
        for k, i in enumerate(pending.tolist()):
            self.queues.setdefault((int(w[i]), int(d[i])), deque()).append(
                (int(o[i]), o_row0 + i, int(ol_first[i]), int(cnt[i]), -1 if no_row0 is None else no_row0 + k))

    def undelivered(self) -> int:
        return sum(len(q) for q in self.queues.values())


def delivery_inputs(n_txn: int, *, seed: int, batch: int, w_lo: int, w_hi: int):
    """The random inputs of ``n_txn`` TPC-C Delivery transactions (TPC-C 2.7.1 [EXT]): home
    warehouse uniform in [w_lo, w_hi), o_carrier_id uniform in [1, 10]."""
    rng = np.random.Generator(np.random.Philox(key=np.array([seed, 1 << 42 | batch], dtype=np.uint64)))
    w = rng.integers(w_lo, w_hi, size=n_txn).astype(np.int32)
    carrier = rng.integers(1, 11, size=n_txn).astype(np.int32)
    return w, carrier


def delivery_batch(state: DeliveryState, w, carrier, clock0: int, step_us: int = 1_000):
    """Row updates of Delivery transactions (TPC-C 2.7.4 [EXT], as SURVEY.md §8(f) NEXT-1 uses it):
    transaction k runs at time ``clock0 + (k+1)*step_us``; for each district d of warehouse
    ``w[k]`` it takes the oldest undelivered order (if any), sets its o_carrier_id to
    ``carrier[k]`` and the ol_delivery_d of each of its lines to the transaction time.
    (The customer balance / delivery count updates touch no column of the hot path.)

    Returns ``{"orders": {"o_carrier_id": (rows, values)},
    "order_line": {"ol_delivery_d": (rows, values)}}`` with rows uint32 (distinct: an order is
    delivered once) and values in the column dtype; plus ``"new_order": {"no_deleted": (rows, 1s)}``
    (the transaction's DELETE FROM new_order) for orders registered with their new_order row."""
    o_rows, o_vals, l_rows, l_vals, n_rows = [], [], [], [], []
    for k in range(len(w)):
        ts = clock0 + (k + 1) * step_us
        for d in range(1, state.districts + 1):
            q = state.queues.get((int(w[k]), d))
            if not q:
                continue
            _, o_row, ol_first, cnt, no_row = q.popleft()
            if no_row >= 0:
                n_rows.append(no_row)
            o_rows.append(o_row)
            o_vals.append(int(carrier[k]))
            l_rows.extend(range(ol_first, ol_first + cnt))
            l_vals.extend([ts] * cnt)
    out = {"orders": {"o_carrier_id": (np.asarray(o_rows, np.uint32), np.asarray(o_vals, np.int32))},
           "order_line": {"ol_delivery_d": (np.asarray(l_rows, np.uint32), np.asarray(l_vals, np.int64))}}
    if n_rows:
        out["new_order"] = {"no_deleted": (np.asarray(n_rows, np.uint32), np.ones(len(n_rows), np.int32))}
    return out


# ------------------------------------------------------- NEXT-3 layout table --
def layout_matrix(nrows: int, ncols: int = 16, *, seed: int = 1, lo: int = -(1 << 20), hi: int = 1 << 20):
    """The logical table of PAPER.md §5.3 (L965-972): ``nrows`` records of ``ncols`` int32
    attributes, values uniform in [lo, hi) from stream Philox([seed, 2^43])."""
    rng = np.random.Generator(np.random.Philox(key=np.array([seed, 1 << 43], dtype=np.uint64)))
    return rng.integers(lo, hi, size=(nrows, ncols), dtype=np.int32)


def encode_layout(m: np.ndarray, layout: str, *, pax_rows: int = 64, col_stride: int = 0) -> np.ndarray:
    """Physical int32 array of logical matrix ``m`` (records x attributes) in ``layout``:
    'nsm' = records back to back (row-major), 'dsm' = attributes back to back (column-major, column
    starts ``col_stride`` elements apart, default nrows), 'pax' = pages of ncols minipages of
    ``pax_rows`` values (the paper's 4 KB pages of 16 x 64; the last page zero-padded)."""
    n, k = m.shape
    if layout == "nsm":
        return np.ascontiguousarray(m).reshape(-1)
    if layout == "dsm":
        stride = col_stride or n
        out = np.zeros((k, stride), np.int32)
        out[:, :n] = m.T
        return out.reshape(-1)
    if layout == "pax":
        pages = -(-n // pax_rows)
        pad = np.zeros((pages * pax_rows, k), np.int32)
        pad[:n] = m
        return np.ascontiguousarray(pad.reshape(pages, pax_rows, k).transpose(0, 2, 1)).reshape(-1)
    raise ValueError(layout)
