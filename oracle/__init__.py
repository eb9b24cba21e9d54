"""CPU oracle for CH-benCHmark Q1 / Q6 / Q18 (and NEXT-2: Q14 / Q12 / Q4 / Q3) — TEST INFRASTRUCTURE ONLY.

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py`` (its ``cpu_baseline``
leg and ``--impl reference``) may import this package. The product path
(``paper_conf_cidr_appuswamykpa17_b200``) never imports it and shares no code with it.

The arithmetic lives in ``oracle.c`` (plain C, single-threaded, row at a time, SQL
three-valued logic; see its header for the passages followed). This module only
compiles it with gcc and marshals numpy arrays through ctypes.

Pins (tests/test_oracle_*.py): SQLite executing the literal CH SQL; brute-force nested
loops over the cartesian product on tiny tables; strict-mode closed forms; a
hand-derived golden fixture (tests/golden/); re-partition and COUNT invariants.
"""
from __future__ import annotations

import ctypes as C
import os
import subprocess

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "oracle.c")
_HDR = os.path.join(_HERE, "oracle.h")
_LIB = os.path.join(_HERE, "liboracle.so")

OR_OVERFLOW = -1
OR_NOMEM = -2


def build(force: bool = False) -> str:
    """Compile liboracle.so with gcc (-O2, no vectorisation tricks needed)."""
    stale = (not os.path.exists(_LIB)) or max(os.path.getmtime(_SRC), os.path.getmtime(_HDR)) > os.path.getmtime(_LIB)
    if force or stale:
        tmp = _LIB + f".{os.getpid()}.tmp"
        subprocess.check_call(["gcc", "-O2", "-std=c11", "-Wall", "-Wextra", "-fPIC", "-shared",
                               "-o", tmp, _SRC])
        os.replace(tmp, _LIB)
    return _LIB


class _OL(C.Structure):
    _fields_ = [("n", C.c_int64), ("w_id", C.c_void_p), ("d_id", C.c_void_p), ("o_id", C.c_void_p),
                ("number", C.c_void_p), ("delivery_d", C.c_void_p), ("quantity", C.c_void_p),
                ("amount", C.c_void_p), ("i_id", C.c_void_p)]


class _O(C.Structure):
    _fields_ = [("n", C.c_int64), ("w_id", C.c_void_p), ("d_id", C.c_void_p), ("o_id", C.c_void_p),
                ("c_id", C.c_void_p), ("ol_cnt", C.c_void_p), ("entry_d", C.c_void_p),
                ("carrier_id", C.c_void_p)]


class _I(C.Structure):
    _fields_ = [("n", C.c_int64), ("i_id", C.c_void_p), ("i_data", C.c_void_p), ("width", C.c_int64)]


class _C(C.Structure):
    _fields_ = [("n", C.c_int64), ("w_id", C.c_void_p), ("d_id", C.c_void_p), ("c_id", C.c_void_p),
                ("c_last", C.c_void_p), ("state", C.c_void_p), ("state_width", C.c_int64)]


class _NO(C.Structure):
    _fields_ = [("n", C.c_int64), ("w_id", C.c_void_p), ("d_id", C.c_void_p), ("o_id", C.c_void_p)]


_lib = None


def _load():
    global _lib
    if _lib is None:
        lib = C.CDLL(build())
        lib.oracle_q6.restype = C.c_int
        lib.oracle_q1.restype = C.c_int64
        lib.oracle_q18.restype = C.c_int64
        lib.oracle_q14.restype = C.c_int
        lib.oracle_q12.restype = C.c_int64
        lib.oracle_q4.restype = C.c_int64
        lib.oracle_q3.restype = C.c_int64
        _lib = lib
    return _lib


def _p(a):
    return a.ctypes.data_as(C.c_void_p) if a is not None else None


def _col(t, name, dtype):
    a = np.ascontiguousarray(t[name], dtype=dtype)
    return a


class _Keep:
    """Holds contiguous copies alive for the duration of a call."""

    def __init__(self):
        self.arrs = []

    def __call__(self, a):
        self.arrs.append(a)
        return _p(a)


def _opt(t, name, dtype, keep):
    return keep(_col(t, name, dtype)) if name in t else None


def _ol_struct(ol, keep):
    n = len(ol["ol_w_id"]) if "ol_w_id" in ol else len(ol["ol_delivery_d"])
    return _OL(n, _opt(ol, "ol_w_id", np.int32, keep), _opt(ol, "ol_d_id", np.int32, keep),
               _opt(ol, "ol_o_id", np.int32, keep), _opt(ol, "ol_number", np.int32, keep),
               keep(_col(ol, "ol_delivery_d", np.int64)), _opt(ol, "ol_quantity", np.int32, keep),
               keep(_col(ol, "ol_amount", np.int64)), _opt(ol, "ol_i_id", np.int32, keep))


def _o_struct(o, keep):
    return _O(len(o["o_w_id"]), keep(_col(o, "o_w_id", np.int32)), keep(_col(o, "o_d_id", np.int32)),
              keep(_col(o, "o_id", np.int32)), _opt(o, "o_c_id", np.int32, keep),
              keep(_col(o, "o_ol_cnt", np.int32)), keep(_col(o, "o_entry_d", np.int64)),
              _opt(o, "o_carrier_id", np.int32, keep))


def _check(st):
    if st == OR_OVERFLOW:
        raise OverflowError("integer overflow in SUM (oracle)")
    if st == OR_NOMEM:
        raise MemoryError("oracle out of memory")


def ts_cmp(op: str, v, c):
    """The oracle's 3-valued timestamp comparison (v is None = SQL NULL): True, False or None."""
    lib = _load()
    code = {">=": 0, "<": 1, ">": 2}[op]
    vv = np.iinfo(np.int64).min if v is None else int(v)
    r = lib.oracle_ts_cmp(C.c_int(code), C.c_int64(vv), C.c_int64(int(c)))
    return {0: False, 1: True, 2: None}[r]


def q6(tables, d_lo, d_hi, q_lo, q_hi):
    """CH Q6. Returns {"revenue": int or None (NULL), "count": qualifying rows}."""
    lib, keep = _load(), _Keep()
    ol = _ol_struct(tables["order_line"], keep)
    rev, isnull, cnt = C.c_int64(), C.c_int32(), C.c_int64()
    _check(lib.oracle_q6(C.byref(ol), C.c_int64(d_lo), C.c_int64(d_hi), C.c_int64(q_lo),
                         C.c_int64(q_hi), C.byref(rev), C.byref(isnull), C.byref(cnt)))
    return {"revenue": None if isnull.value else rev.value, "count": cnt.value}


def q1(tables, cutoff):
    """CH Q1. Returns a dict of numpy columns ordered by ol_number."""
    lib, keep = _load(), _Keep()
    ol = _ol_struct(tables["order_line"], keep)
    cap = 64
    while True:
        out = {"ol_number": np.zeros(cap, np.int32), "sum_qty": np.zeros(cap, np.int64),
               "sum_amount": np.zeros(cap, np.int64), "avg_qty": np.zeros(cap, np.float64),
               "avg_amount": np.zeros(cap, np.float64), "count_order": np.zeros(cap, np.int64)}
        n = lib.oracle_q1(C.byref(ol), C.c_int64(cutoff), C.c_int64(cap),
                          _p(out["ol_number"]), _p(out["sum_qty"]), _p(out["sum_amount"]),
                          _p(out["avg_qty"]), _p(out["avg_amount"]), _p(out["count_order"]))
        _check(n if n < 0 else 0)
        if n <= cap:
            return {k: v[:n] for k, v in out.items()}
        cap = n


Q18_COLUMNS = [("c_last", np.int32), ("c_id", np.int32), ("o_id", np.int32), ("o_entry_d", np.int64),
               ("o_ol_cnt", np.int32), ("amount_sum", np.int64), ("o_w_id", np.int32),
               ("o_d_id", np.int32)]


def q18(tables, having):
    """CH Q18 (customer ⋈ orders ⋈ order_line). Returns numpy columns in ORDER BY order."""
    lib, keep = _load(), _Keep()
    ol = _ol_struct(tables["order_line"], keep)
    o, c = tables["orders"], tables["customer"]
    os_ = _o_struct(o, keep)
    cs = _C(len(c["c_w_id"]), keep(_col(c, "c_w_id", np.int32)), keep(_col(c, "c_d_id", np.int32)),
            keep(_col(c, "c_id", np.int32)), keep(_col(c, "c_last", np.int32)), None, 0)
    cap = max(1, len(o["o_w_id"]))
    while True:
        out = {k: np.zeros(cap, dt) for k, dt in Q18_COLUMNS}
        n = lib.oracle_q18(C.byref(cs), C.byref(os_), C.byref(ol), C.c_int64(having), C.c_int64(cap),
                           *[_p(out[k]) for k, _ in Q18_COLUMNS])
        _check(n if n < 0 else 0)
        if n <= cap:
            return {k: v[:n] for k, v in out.items()}
        cap = n


def apply_updates(tables, updates):
    """The snapshot after in-place updates: for every
    ``updates[table][column] = (rows, values)``, row ``rows[i]`` of that column holds
    ``values[i]``; every other value is unchanged. This is the plain definition of the paper's
    copy-on-write update as seen by a later snapshot ("updates ... shadow-copy the pages they
    touch"); row ids are distinct. Returns new tables; the input tables (the
    previous snapshot) are not modified."""
    out = {t: dict(cols) for t, cols in tables.items()}
    for t, per_col in updates.items():
        for c, (rows, values) in per_col.items():
            col = np.array(out[t][c], copy=True)
            col[np.asarray(rows, dtype=np.int64)] = values
            out[t][c] = col
    return out


def q14(tables, d_lo, d_hi, prefix=b"PR"):
    """CH Q14 (order_line ⋈ item): {"promo_revenue": float or None (NULL), "sum_promo",
    "sum_amount", "count"} — promo_revenue = 100.0 * sum_promo / (100.0 + sum_amount) (cents)."""
    lib, keep = _load(), _Keep()
    ol = _ol_struct(tables["order_line"], keep)
    it = tables["item"]
    data = np.ascontiguousarray(np.asarray(it["i_data"], dtype="S50"))
    its = _I(len(it["i_id"]), keep(_col(it, "i_id", np.int32)), keep(data), 50)
    promo, isnull = C.c_double(), C.c_int32()
    sp, sa, cnt = C.c_int64(), C.c_int64(), C.c_int64()
    _check(lib.oracle_q14(C.byref(ol), C.byref(its), C.c_int64(d_lo), C.c_int64(d_hi),
                          C.c_char_p(bytes(prefix)), C.byref(promo), C.byref(isnull), C.byref(sp),
                          C.byref(sa), C.byref(cnt)))
    return {"promo_revenue": None if isnull.value else promo.value, "sum_promo": sp.value,
            "sum_amount": sa.value, "count": cnt.value}


def _small_groups(fn, names, dtypes):
    cap = 64
    while True:
        out = {k: np.zeros(cap, dt) for k, dt in zip(names, dtypes)}
        n = fn(cap, *[_p(out[k]) for k in names])
        _check(n if n < 0 else 0)
        if n <= cap:
            return {k: v[:n] for k, v in out.items()}
        cap = n


def q12(tables, d_hi):
    """CH Q12 (orders ⋈ order_line): columns o_ol_cnt, high_line_count, low_line_count."""
    lib, keep = _load(), _Keep()
    ol = _ol_struct(tables["order_line"], keep)
    o = _o_struct(tables["orders"], keep)
    return _small_groups(lambda cap, *ps: lib.oracle_q12(C.byref(o), C.byref(ol), C.c_int64(d_hi),
                                                         C.c_int64(cap), *ps),
                         ["o_ol_cnt", "high_line_count", "low_line_count"], [np.int32, np.int64, np.int64])


def q4(tables, e_lo, e_hi):
    """CH Q4 (orders semi-join order_line): columns o_ol_cnt, order_count."""
    lib, keep = _load(), _Keep()
    ol = _ol_struct(tables["order_line"], keep)
    o = _o_struct(tables["orders"], keep)
    return _small_groups(lambda cap, *ps: lib.oracle_q4(C.byref(o), C.byref(ol), C.c_int64(e_lo),
                                                        C.c_int64(e_hi), C.c_int64(cap), *ps),
                         ["o_ol_cnt", "order_count"], [np.int32, np.int64])


Q3_COLUMNS = [("ol_o_id", np.int32), ("ol_w_id", np.int32), ("ol_d_id", np.int32),
              ("revenue", np.int64), ("o_entry_d", np.int64)]


def q3(tables, entry_lo, prefix=b"A"):
    """CH Q3 (customer ⋈ new_order ⋈ orders ⋈ order_line, GROUP BY, ORDER BY revenue DESC,
    o_entry_d). Returns numpy columns ol_o_id, ol_w_id, ol_d_id, revenue, o_entry_d in order."""
    lib, keep = _load(), _Keep()
    ol = _ol_struct(tables["order_line"], keep)
    os_ = _o_struct(tables["orders"], keep)
    c, no = tables["customer"], tables["new_order"]
    state = np.ascontiguousarray(np.asarray(c["c_state"], dtype="S2"))
    cs = _C(len(c["c_w_id"]), keep(_col(c, "c_w_id", np.int32)), keep(_col(c, "c_d_id", np.int32)),
            keep(_col(c, "c_id", np.int32)), None, keep(state), 2)
    ns = _NO(len(no["no_w_id"]), keep(_col(no, "no_w_id", np.int32)),
             keep(_col(no, "no_d_id", np.int32)), keep(_col(no, "no_o_id", np.int32)))
    cap = max(1, len(no["no_w_id"]))
    while True:
        out = {k: np.zeros(cap, dt) for k, dt in Q3_COLUMNS}
        n = lib.oracle_q3(C.byref(cs), C.byref(ns), C.byref(os_), C.byref(ol), C.c_int64(entry_lo),
                          C.c_char_p(bytes(prefix)), C.c_int64(cap), *[_p(out[k]) for k, _ in Q3_COLUMNS])
        _check(n if n < 0 else 0)
        if n <= cap:
            return {k: v[:n] for k, v in out.items()}
        cap = n


LAYOUTS = {"dsm": 1, "pax": 2, "nsm": 3}


def layout_sum(data, layout, nrows, ncols, columns, *, col_stride=0, pax_rows=64):
    """NEXT-3: SUM(col_c1 + ... + col_cN) over the physical int32 table ``data`` in ``layout``
    ('dsm' / 'pax' / 'nsm'). Returns the sum, or None (NULL) for no rows."""
    lib = _load()
    lib.oracle_layout_sum.restype = C.c_int
    a = np.ascontiguousarray(data, dtype=np.int32)
    mask = 0
    for c in columns:
        mask |= 1 << int(c)
    out, isnull = C.c_int64(), C.c_int32()
    _check(lib.oracle_layout_sum(_p(a), C.c_int(LAYOUTS[layout]), C.c_int64(nrows), C.c_int64(ncols),
                                 C.c_int64(col_stride or nrows), C.c_int64(pax_rows), C.c_uint64(mask),
                                 C.byref(out), C.byref(isnull)))
    return None if isnull.value else out.value
