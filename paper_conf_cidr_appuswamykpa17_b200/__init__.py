"""B200-native OLAP hot path of an H2TAP engine (Appuswamy et al., CIDR 2017).

Thin Python binding of the C ABI in ``include/h2tap.h`` (``libh2tap.so``, built in-tree by
``_build.py`` for sm_100a). Every function here only marshals arguments: the snapshot store,
the query kernels, the cross-GPU merge (peer-memory kernels) and the finalisation all run in
the CUDA library. There is
no CPU fallback — importing this package fails loudly when the library is missing.

Names mirror the ABI: ``h2tap_open``, ``h2tap_load_snapshot``, ``h2tap_sync``,
``h2tap_refresh``, ``h2tap_refresh_rows``, ``h2tap_get_store_stats``,
``h2tap_run_query``, ``h2tap_free``, ``h2tap_close``, ``h2tap_last_error``,
``h2tap_peer_handle``, ``h2tap_peer_connect``, ``h2tap_peer_connect_local``,
``h2tap_compute_stream``, ``h2tap_c_last_name``.
"""
from __future__ import annotations

import ctypes as C
import os

import numpy as np

_PKG = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.path.join(_PKG, "libh2tap.so")
if os.environ.get("H2TAP_LIB"):  # an A/B build variant (scripts/build_variants.py), never the default
    LIB_PATH = os.environ["H2TAP_LIB"]

if not os.path.exists(LIB_PATH):
    raise ImportError(
        f"{LIB_PATH} is missing: build it with `python -m paper_conf_cidr_appuswamykpa17_b200._build` "
        "(or __graft_entry__.build()). There is no CPU fallback.")

_lib = C.CDLL(LIB_PATH)

# ------------------------------------------------------------------ ABI types --
H2TAP_OK, H2TAP_EINVAL, H2TAP_ESTALE, H2TAP_ENOMEM = 0, -1, -2, -3
H2TAP_ECUDA, H2TAP_EPEER, H2TAP_EPLAN, H2TAP_EDUPKEY, H2TAP_ESHAPE = -4, -5, -6, -7, -8
STATUS_NAMES = {0: "OK", -1: "EINVAL", -2: "ESTALE", -3: "ENOMEM", -4: "ECUDA", -5: "EPEER",
                -6: "EPLAN", -7: "EDUPKEY", -8: "ESHAPE", -9: "EOVERFLOW"}
H2TAP_I32, H2TAP_I64, H2TAP_F64 = 1, 2, 3
H2TAP_T_ORDER_LINE, H2TAP_T_ORDERS, H2TAP_T_CUSTOMER, H2TAP_T_ITEM, H2TAP_T_NEW_ORDER = 1, 2, 3, 4, 5
H2TAP_Q1, H2TAP_Q6, H2TAP_Q18 = 1, 6, 18
H2TAP_Q3, H2TAP_Q4, H2TAP_Q12, H2TAP_Q14 = 3, 4, 12, 14  # NEXT-2 CH queries
H2TAP_FULL_RELOAD = 1
H2TAP_DSM, H2TAP_PAX, H2TAP_NSM = 1, 2, 3  # NEXT-3 layouts (§5.3)
H2TAP_LOAD_ASYNC = 1
H2TAP_LOAD_ZERO_COPY = 2  # NEXT-4: kernels read the caller's pinned host columns over PCIe
H2TAP_LOAD_BORROW = 4  # with ASYNC: pinned buffers lent to the DMA until the epoch is published
H2TAP_RESULT_DEVICE = 1
H2TAP_QUERY_PROFILE = 2
H2TAP_QUERY_HASH_JOIN = 4

_DT = {H2TAP_I32: np.int32, H2TAP_I64: np.int64, H2TAP_F64: np.float64}

# Column ids per table, in header order (h2tap.h), keyed by the generator's column names.
SCHEMA = {
    "order_line": (H2TAP_T_ORDER_LINE, [
        ("ol_w_id", H2TAP_I32), ("ol_d_id", H2TAP_I32), ("ol_o_id", H2TAP_I32),
        ("ol_number", H2TAP_I32), ("ol_i_id", H2TAP_I32), ("ol_supply_w_id", H2TAP_I32),
        ("ol_delivery_d", H2TAP_I64), ("ol_quantity", H2TAP_I32), ("ol_amount", H2TAP_I64)]),
    "orders": (H2TAP_T_ORDERS, [
        ("o_w_id", H2TAP_I32), ("o_d_id", H2TAP_I32), ("o_id", H2TAP_I32), ("o_c_id", H2TAP_I32),
        ("o_ol_cnt", H2TAP_I32), ("o_carrier_id", H2TAP_I32), ("o_all_local", H2TAP_I32),
        ("o_entry_d", H2TAP_I64)]),
    "customer": (H2TAP_T_CUSTOMER, [
        ("c_w_id", H2TAP_I32), ("c_d_id", H2TAP_I32), ("c_id", H2TAP_I32), ("c_last", H2TAP_I32),
        ("c_state_p2", H2TAP_I32)]),
    "item": (H2TAP_T_ITEM, [("i_id", H2TAP_I32), ("i_price", H2TAP_I64), ("i_data_p2", H2TAP_I32)]),
    "new_order": (H2TAP_T_NEW_ORDER, [("no_w_id", H2TAP_I32), ("no_d_id", H2TAP_I32), ("no_o_id", H2TAP_I32),
                                      ("no_deleted", H2TAP_I32)]),
}


class h2tap_column(C.Structure):
    _fields_ = [("column_id", C.c_uint32), ("type", C.c_uint32), ("host_data", C.c_void_p)]


class h2tap_table(C.Structure):
    _fields_ = [("table_id", C.c_uint32), ("ncols", C.c_uint32), ("cols", C.POINTER(h2tap_column)),
                ("row_count", C.c_uint64), ("first_row", C.c_uint64), ("flags", C.c_uint32)]


class h2tap_field(C.Structure):
    _fields_ = [("column_id", C.c_uint32), ("type", C.c_uint32), ("offset", C.c_uint32)]


class h2tap_row_table(C.Structure):
    _fields_ = [("table_id", C.c_uint32), ("nfields", C.c_uint32), ("fields", C.POINTER(h2tap_field)),
                ("records", C.c_void_p), ("record_size", C.c_uint64), ("row_count", C.c_uint64),
                ("first_row", C.c_uint64), ("flags", C.c_uint32)]


class h2tap_update(C.Structure):
    _fields_ = [("table_id", C.c_uint32), ("column_id", C.c_uint32), ("type", C.c_uint32),
                ("n", C.c_uint64), ("row_ids", C.c_void_p), ("values", C.c_void_p)]


class h2tap_store_stats(C.Structure):
    _fields_ = [("published_epoch", C.c_uint64), ("refreshes", C.c_uint64),
                ("rows_appended", C.c_uint64), ("rows_updated", C.c_uint64),
                ("cow_pages_copied", C.c_uint64), ("cow_full_copies", C.c_uint64),
                ("device_bytes", C.c_uint64), ("last_load_ms", C.c_double),
                ("last_update_h2d_ms", C.c_double), ("last_update_ms", C.c_double)]


class h2tap_config(C.Structure):
    _fields_ = [("device", C.c_int), ("rank", C.c_int), ("world", C.c_int),
                ("peer_heap_bytes", C.c_uint64)]


class h2tap_query(C.Structure):
    _fields_ = [("plan_id", C.c_uint32), ("nparams", C.c_uint32), ("params", C.POINTER(C.c_int64)),
                ("flags", C.c_uint32)]


class h2tap_result(C.Structure):
    _fields_ = [("epoch", C.c_uint64), ("nrows", C.c_uint64), ("ncols", C.c_uint32),
                ("on_device", C.c_uint32), ("names", C.POINTER(C.c_char_p)),
                ("types", C.POINTER(C.c_uint32)), ("cols", C.POINTER(C.c_void_p)),
                ("nulls", C.POINTER(C.POINTER(C.c_uint8))), ("rows_scanned", C.c_uint64),
                ("device_ms", C.c_double), ("e2e_ms", C.c_double), ("nkernels", C.c_uint32),
                ("kernel_names", C.POINTER(C.c_char_p)), ("kernel_ms", C.POINTER(C.c_double)),
                ("kernel_launches", C.c_uint64), ("plan_flags", C.c_uint32),
                ("row_offset", C.c_uint64), ("total_rows", C.c_uint64)]


class h2tap_layout_table(C.Structure):
    _fields_ = [("data", C.c_void_p), ("layout", C.c_uint32), ("ncols", C.c_uint32),
                ("nrows", C.c_uint64), ("col_stride", C.c_uint64), ("pax_rows", C.c_uint32)]


_P = C.c_void_p
_lib.h2tap_layout_sum.argtypes = [_P, C.POINTER(h2tap_layout_table), C.c_uint64, C.POINTER(C.c_int64),
                                  C.POINTER(C.c_int32), C.POINTER(C.c_double)]
_lib.h2tap_open.argtypes = [C.POINTER(h2tap_config), C.POINTER(_P)]
_lib.h2tap_load_snapshot_ex.argtypes = [_P, C.POINTER(h2tap_table), C.c_uint32, C.c_uint64, C.c_uint32]
_lib.h2tap_load_snapshot.argtypes = [_P, C.POINTER(h2tap_table), C.c_uint32, C.c_uint64]
_lib.h2tap_sync.argtypes = [_P, C.POINTER(C.c_uint64)]
_lib.h2tap_reserve.argtypes = [_P, C.c_uint32, C.c_uint64]
_lib.h2tap_load_snapshot_rows.argtypes = [_P, C.POINTER(h2tap_row_table), C.c_uint32, C.c_uint64,
                                          C.c_uint32]
_lib.h2tap_refresh.argtypes = [_P, C.POINTER(h2tap_table), C.c_uint32, C.POINTER(h2tap_update),
                               C.c_uint32, C.c_uint64, C.c_uint32]
_lib.h2tap_refresh_rows.argtypes = [_P, C.POINTER(h2tap_row_table), C.c_uint32,
                                    C.POINTER(h2tap_update), C.c_uint32, C.c_uint64, C.c_uint32]
_lib.h2tap_get_store_stats.argtypes = [_P, C.POINTER(h2tap_store_stats)]
_lib.h2tap_run_query_ex.argtypes = [_P, C.c_uint32, C.POINTER(C.c_int64), C.c_uint32, C.c_uint32,
                                    C.POINTER(C.POINTER(h2tap_result))]
_lib.h2tap_run_query.argtypes = [_P, C.c_uint32, C.POINTER(C.c_int64), C.c_uint32,
                                 C.POINTER(C.POINTER(h2tap_result))]
_lib.h2tap_run_queries.argtypes = [_P, C.POINTER(h2tap_query), C.c_uint32,
                                   C.POINTER(C.POINTER(h2tap_result))]
_lib.h2tap_last_batch_ms.argtypes = [_P, C.POINTER(C.c_double)]
_lib.h2tap_free.argtypes = [C.POINTER(h2tap_result)]
_lib.h2tap_free.restype = None
_lib.h2tap_close.argtypes = [_P]
_lib.h2tap_close.restype = None
_lib.h2tap_last_error.restype = C.c_char_p
_lib.h2tap_peer_handle.argtypes = [_P, _P]
_lib.h2tap_peer_connect.argtypes = [_P, _P, C.c_uint32]
_lib.h2tap_peer_connect_local.argtypes = [C.POINTER(_P), C.c_uint32]
_lib.h2tap_compute_stream.argtypes = [_P, C.POINTER(_P)]
_lib.h2tap_c_last_name.argtypes = [C.c_int32, C.c_char_p, C.c_size_t]
for _f in ("h2tap_open", "h2tap_load_snapshot_ex", "h2tap_load_snapshot", "h2tap_load_snapshot_rows",
           "h2tap_reserve", "h2tap_refresh", "h2tap_refresh_rows", "h2tap_get_store_stats",
           "h2tap_sync",
           "h2tap_run_query_ex", "h2tap_run_query", "h2tap_run_queries", "h2tap_peer_handle",
           "h2tap_peer_connect", "h2tap_peer_connect_local", "h2tap_compute_stream", "h2tap_layout_sum",
           "h2tap_last_batch_ms"):
    getattr(_lib, _f).restype = C.c_int

ABI_SYMBOLS = ["h2tap_open", "h2tap_load_snapshot", "h2tap_load_snapshot_ex",
               "h2tap_load_snapshot_rows", "h2tap_reserve", "h2tap_refresh", "h2tap_refresh_rows",
               "h2tap_get_store_stats", "h2tap_sync",
               "h2tap_run_query", "h2tap_run_query_ex", "h2tap_run_queries", "h2tap_free", "h2tap_close",
               "h2tap_last_error", "h2tap_peer_handle", "h2tap_peer_connect",
               "h2tap_peer_connect_local", "h2tap_compute_stream",
               "h2tap_c_last_name", "h2tap_layout_sum", "h2tap_last_batch_ms"]


class H2tapError(RuntimeError):
    def __init__(self, status, msg):
        super().__init__(f"H2TAP_{STATUS_NAMES.get(status, status)}: {msg}")
        self.status = status


def h2tap_last_error() -> str:
    return (_lib.h2tap_last_error() or b"").decode()


def _check(st):
    if st != H2TAP_OK:
        raise H2tapError(st, h2tap_last_error())


# ------------------------------------------------------------------ wrappers --
class Engine:
    """Handle of one engine (one GPU rank). Use h2tap_close() or the context manager."""

    def __init__(self, handle, device, rank, world):
        self.handle, self.device, self.rank, self.world = handle, device, rank, world

    def __enter__(self):
        return self

    def __exit__(self, *exc):
        h2tap_close(self)


def h2tap_open(device: int = 0, rank: int = 0, world: int = 1, peer_heap_bytes: int = 0) -> Engine:
    cfg = h2tap_config(device, rank, world, peer_heap_bytes)
    h = _P()
    _check(_lib.h2tap_open(C.byref(cfg), C.byref(h)))
    return Engine(h, device, rank, world)


def h2tap_peer_handle(engine: Engine) -> bytes:
    """This rank's 64-byte CUDA IPC handle of its peer segment (world > 1)."""
    buf = C.create_string_buffer(64)
    _check(_lib.h2tap_peer_handle(engine.handle, C.cast(buf, _P)))
    return buf.raw


def h2tap_peer_connect(engine: Engine, handles) -> None:
    """Map every rank's peer segment (``handles``: the world's 64-byte handles in rank order)."""
    blob = b"".join(bytes(h) for h in handles)
    buf = C.create_string_buffer(blob, len(blob))
    _check(_lib.h2tap_peer_connect(engine.handle, C.cast(buf, _P), len(handles)))


def h2tap_peer_connect_local(engines) -> None:
    """Connect engines of ONE process (engines[k] has rank k); they may share a device."""
    arr = (_P * len(engines))(*[e.handle for e in engines])
    _check(_lib.h2tap_peer_connect_local(arr, len(engines)))


def open_local_group(world: int, device: int = 0, peer_heap_bytes: int = 0) -> list:
    """``world`` engines (ranks 0..world-1) on ``device`` in this process, peer-connected: the whole
    multi-GPU path with merges through one device's memory. Their collective calls must be issued
    concurrently (one host thread per engine, e.g. :func:`run_collective`)."""
    engines = [h2tap_open(device, k, world, peer_heap_bytes) for k in range(world)]
    try:
        h2tap_peer_connect_local(engines)
    except BaseException:
        for e in engines:
            h2tap_close(e)
        raise
    return engines


def run_collective(engines, fn):
    """Call ``fn(engine)`` for every engine concurrently (one thread each: collectives need every
    rank's launch); returns the results in rank order, re-raising the first exception."""
    import threading
    out, err = [None] * len(engines), [None] * len(engines)

    def work(k):
        try:
            out[k] = fn(engines[k])
        except BaseException as x:  # noqa: BLE001 (re-raised below)
            err[k] = x

    ts = [threading.Thread(target=work, args=(k,)) for k in range(len(engines))]
    for t in ts:
        t.start()
    for t in ts:
        t.join()
    for x in err:
        if x is not None:
            raise x
    return out


def connect_torch_group(engine: Engine, group=None) -> None:
    """Multi-process bootstrap: exchange the ranks' peer handles over an initialised
    torch.distributed process group (plumbing only), then map the segments."""
    import torch.distributed as dist
    handles = [None] * engine.world
    dist.all_gather_object(handles, h2tap_peer_handle(engine), group=group)
    h2tap_peer_connect(engine, handles)


def h2tap_close(engine: Engine) -> None:
    if engine is not None and engine.handle:
        _lib.h2tap_close(engine.handle)
        engine.handle = None


def _host_ptr(a, want_dtype, name):
    """Host pointer of a contiguous numpy array or CPU torch tensor (pinned or not)."""
    if hasattr(a, "data_ptr") and hasattr(a, "is_cuda"):
        if a.is_cuda:
            raise ValueError(f"{name}: column buffers are host memory (the snapshot is refreshed H2D)")
        if not a.is_contiguous() or a.element_size() != np.dtype(want_dtype).itemsize:
            raise ValueError(f"{name}: needs a contiguous {np.dtype(want_dtype).name} tensor")
        return a.data_ptr(), a, a.numel()
    arr = np.ascontiguousarray(a)
    if arr.dtype != want_dtype:
        raise ValueError(f"{name}: dtype {arr.dtype}, schema wants {np.dtype(want_dtype).name}")
    return arr.ctypes.data, arr, arr.size


def _column_tables(tables, full_reload, first_row):
    first_row = first_row or {}
    keep, tabs, colarrs = [], [], []
    for tname, cols in tables.items():
        tid, schema = SCHEMA[tname]
        ids = {n: (i, t) for i, (n, t) in enumerate(schema)}
        carr = (h2tap_column * len(cols))()
        nrows = None
        for k, (cname, a) in enumerate(cols.items()):
            cid, ty = ids[cname]
            ptr, obj, n = _host_ptr(a, _DT[ty], f"{tname}.{cname}")
            keep.append(obj)
            if nrows is None:
                nrows = n
            elif n != nrows:
                raise ValueError(f"{tname}: columns have different lengths ({n} vs {nrows})")
            carr[k] = h2tap_column(cid, ty, ptr)
        full = full_reload if isinstance(full_reload, bool) else tname in full_reload
        fr = 0 if full else int(first_row.get(tname, 0))
        colarrs.append(carr)
        tabs.append(h2tap_table(tid, len(cols), carr, fr + (nrows or 0), fr,
                                H2TAP_FULL_RELOAD if full else 0))
    return (h2tap_table * len(tabs))(*tabs), len(tabs), keep + colarrs


def _updates(updates):
    """{table: {column: (row_ids, values)}} -> h2tap_update array (+ objects to keep alive)."""
    ups, keep = [], []
    for tname, per_col in (updates or {}).items():
        tid, schema = SCHEMA[tname]
        ids = {n: (i, t) for i, (n, t) in enumerate(schema)}
        for cname, (rows, vals) in per_col.items():
            cid, ty = ids[cname]
            rp, robj, nr = _host_ptr(rows, np.uint32, f"{tname}.{cname} row ids")
            vp, vobj, nv = _host_ptr(vals, _DT[ty], f"{tname}.{cname} values")
            if nr != nv:
                raise ValueError(f"{tname}.{cname}: {nr} row ids but {nv} values")
            keep += [robj, vobj]
            ups.append(h2tap_update(tid, cid, ty, nr, rp if nr else None, vp if nv else None))
    return (h2tap_update * max(len(ups), 1))(*ups), len(ups), keep


def h2tap_load_snapshot(engine: Engine, tables: dict, epoch: int, *, flags: int = 0,
                        full_reload=True, first_row: dict | None = None) -> None:
    """Refresh the device snapshot to ``epoch``.

    ``tables``: {table_name: {column_name: array}} with the generator's names. Each array holds
    rows [first_row, row_count) of its column. ``full_reload`` (bool, or a set of table names)
    replaces those tables; other tables are appended to (``first_row[table]`` = rows already
    loaded). ``flags``: H2TAP_LOAD_ASYNC to return before the epoch is published.
    """
    tarr, nt, keep = _column_tables(tables, full_reload, first_row)
    _check(_lib.h2tap_load_snapshot_ex(engine.handle, tarr, nt, epoch, flags))
    del keep


def h2tap_refresh(engine: Engine, tables: dict | None, updates: dict | None, epoch: int, *,
                  flags: int = 0, full_reload=False, first_row: dict | None = None) -> None:
    """One new epoch = appends / reloads of ``tables`` (as h2tap_load_snapshot; default append)
    then in-place ``updates`` = {table: {column: (row_ids uint32, values)}} (copy-on-write)."""
    tarr, nt, keep = _column_tables(tables or {}, full_reload, first_row)
    uarr, nu, ukeep = _updates(updates)
    _check(_lib.h2tap_refresh(engine.handle, tarr, nt, uarr, nu, epoch, flags))
    del keep, ukeep


def h2tap_get_store_stats(engine: Engine) -> dict:
    """Snapshot-store counters and the last refresh's copy-stream times (h2tap_store_stats)."""
    st = h2tap_store_stats()
    _check(_lib.h2tap_get_store_stats(engine.handle, C.byref(st)))
    return {name: getattr(st, name) for name, _ in h2tap_store_stats._fields_}


def _row_tables(tables, full_reload, first_row, columns):
    first_row = first_row or {}
    keep, tabs = [], []
    for tname, rec in tables.items():
        tid, schema = SCHEMA[tname]
        rec = np.ascontiguousarray(rec)
        want = columns.get(tname) if columns else None
        fields = []
        for cid, (cname, ty) in enumerate(schema):
            if cname not in (rec.dtype.fields or {}) or (want is not None and cname not in want):
                continue
            fdt, off = rec.dtype.fields[cname][:2]
            if fdt != np.dtype(_DT[ty]):
                raise ValueError(f"{tname}.{cname}: record field {fdt}, schema {np.dtype(_DT[ty])}")
            fields.append(h2tap_field(cid, ty, off))
        farr = (h2tap_field * len(fields))(*fields)
        keep += [rec, farr]
        full = full_reload if isinstance(full_reload, bool) else tname in full_reload
        fr = 0 if full else int(first_row.get(tname, 0))
        tabs.append(h2tap_row_table(tid, len(fields), farr, rec.ctypes.data if len(rec) else None,
                                    rec.dtype.itemsize, fr + len(rec), fr,
                                    H2TAP_FULL_RELOAD if full else 0))
    return (h2tap_row_table * len(tabs))(*tabs), len(tabs), keep


def h2tap_load_snapshot_rows(engine: Engine, tables: dict, epoch: int, *, flags: int = 0,
                             full_reload=True, first_row: dict | None = None,
                             columns: dict | None = None) -> None:
    """Refresh from a host ROW store: ``tables`` = {table_name: numpy structured array of NSM
    records}. ``columns`` optionally restricts the extracted fields per table (default: every
    schema field present in the record dtype). Other arguments as h2tap_load_snapshot."""
    tarr, nt, keep = _row_tables(tables, full_reload, first_row, columns)
    _check(_lib.h2tap_load_snapshot_rows(engine.handle, tarr, nt, epoch, flags))
    del keep


def h2tap_refresh_rows(engine: Engine, tables: dict | None, updates: dict | None, epoch: int, *,
                       flags: int = 0, full_reload=False, first_row: dict | None = None,
                       columns: dict | None = None) -> None:
    """h2tap_load_snapshot_rows (default append) plus in-place ``updates`` in the same epoch."""
    tarr, nt, keep = _row_tables(tables or {}, full_reload, first_row, columns)
    uarr, nu, ukeep = _updates(updates)
    _check(_lib.h2tap_refresh_rows(engine.handle, tarr, nt, uarr, nu, epoch, flags))
    del keep, ukeep


def h2tap_reserve(engine: Engine, table: str, rows: int) -> None:
    """Pre-size a loaded table's columns for ``rows`` rows (appends then never reallocate)."""
    _check(_lib.h2tap_reserve(engine.handle, SCHEMA[table][0], rows))


def h2tap_last_batch_ms(engine: Engine) -> float:
    """Device time (CUDA events, ms) of the engine's last completed h2tap_run_queries batch."""
    ms = C.c_double()
    _check(_lib.h2tap_last_batch_ms(engine.handle, C.byref(ms)))
    return ms.value


def h2tap_sync(engine: Engine) -> int:
    ep = C.c_uint64()
    _check(_lib.h2tap_sync(engine.handle, C.byref(ep)))
    return ep.value


class _DevArray:
    """__cuda_array_interface__ view of a device result column (for torch.as_tensor)."""

    def __init__(self, ptr, n, dtype):
        self.__cuda_array_interface__ = {"shape": (n,), "typestr": np.dtype(dtype).str,
                                         "data": (ptr or 0, False), "version": 3, "strides": None}


class Result:
    """A query result. ``columns``: name -> numpy array (zero-copy view of library-owned pinned
    memory, valid until h2tap_free) or, for device results, a __cuda_array_interface__ object.
    ``nulls``: name -> uint8 array, only for columns that can hold NULL. Columns, nulls and the
    per-kernel times are materialised on first access (the scalar fields are read eagerly)."""

    def __init__(self, ptr):
        self._ptr = ptr
        r = ptr.contents
        self.epoch, self.nrows, self.on_device = r.epoch, r.nrows, bool(r.on_device)
        self.rows_scanned, self.device_ms, self.e2e_ms = r.rows_scanned, r.device_ms, r.e2e_ms
        self.kernel_launches = r.kernel_launches
        self.plan_flags = r.plan_flags
        self.row_offset, self.total_rows = r.row_offset, r.total_rows
        self._columns = self._nulls = self._kernels = None

    def _materialise(self):
        r = self._ptr.contents
        cols, nulls = {}, {}
        for i in range(r.ncols):
            name = r.names[i].decode()
            dt = _DT[r.types[i]]
            p = r.cols[i]
            if self.on_device:
                cols[name] = _DevArray(p, self.nrows, dt)
            elif self.nrows:
                cols[name] = np.ctypeslib.as_array(C.cast(p, C.POINTER(np.ctypeslib.as_ctypes_type(dt))), (self.nrows,))
            else:
                cols[name] = np.zeros(0, dt)
            if bool(r.nulls[i]):
                nulls[name] = np.ctypeslib.as_array(r.nulls[i], (self.nrows,)).copy()
        self._columns, self._nulls = cols, nulls

    @property
    def columns(self):
        if self._columns is None:
            if not self._ptr:
                return {}
            self._materialise()
        return self._columns

    @property
    def nulls(self):
        if self._nulls is None:
            if not self._ptr:
                return {}
            self._materialise()
        return self._nulls

    @property
    def kernels(self):
        """[(kernel name, CUDA-event ms)] recorded with H2TAP_QUERY_PROFILE."""
        if self._kernels is None:
            r = self._ptr.contents
            self._kernels = [(r.kernel_names[i].decode(), r.kernel_ms[i]) for i in range(r.nkernels)]
        return self._kernels

    def to_numpy(self) -> dict:
        """Copy every column to a fresh host numpy array (device results via torch)."""
        if not self.on_device:
            return {k: np.array(v, copy=True) for k, v in self.columns.items()}
        import torch
        return {k: torch.as_tensor(v, device="cuda").cpu().numpy() if self.nrows else
                np.zeros(0, np.dtype(v.__cuda_array_interface__["typestr"]))
                for k, v in self.columns.items()}

    def free(self):
        h2tap_free(self)


def h2tap_run_query(engine: Engine, plan: int, params=None, *, flags: int = 0) -> Result:
    """Run plan H2TAP_Q1 / H2TAP_Q6 / H2TAP_Q18 (params: list of int64, None = CH defaults)."""
    params = list(params or [])
    parr = (C.c_int64 * max(1, len(params)))(*params)
    out = C.POINTER(h2tap_result)()
    _check(_lib.h2tap_run_query_ex(engine.handle, plan, parr, len(params), flags, C.byref(out)))
    return Result(out)


def h2tap_run_queries(engine: Engine, queries) -> list:
    """Run a batch on one published epoch: ``queries`` = [(plan, params or None, flags), ...].
    All plans are enqueued back to back and the library synchronises once."""
    n = len(queries)
    qarr = (h2tap_query * max(1, n))()
    keep = []
    for i, (plan, params, flags) in enumerate(queries):
        params = list(params or [])
        parr = (C.c_int64 * max(1, len(params)))(*params)
        keep.append(parr)
        qarr[i] = h2tap_query(plan, len(params), parr, flags)
    outs = (C.POINTER(h2tap_result) * max(1, n))()
    _check(_lib.h2tap_run_queries(engine.handle, qarr, n, outs))
    return [Result(outs[i]) for i in range(n)]


def h2tap_free(result: Result) -> None:
    if result is not None and result._ptr:
        _lib.h2tap_free(result._ptr)
        result._ptr = None
        result._columns = {}


def h2tap_compute_stream(engine: Engine) -> int:
    s = _P()
    _check(_lib.h2tap_compute_stream(engine.handle, C.byref(s)))
    return s.value or 0


def h2tap_c_last_name(code: int) -> str:
    buf = C.create_string_buffer(32)
    n = _lib.h2tap_c_last_name(code, buf, 32)
    if n < 0:
        raise ValueError(f"c_last code {code} outside 0..999")
    return buf.value.decode()


HOT_PATH_PLANS = (H2TAP_Q1, H2TAP_Q6, H2TAP_Q18)  # BASELINE north_star


def plan_columns():
    """Columns each plan reads (what h2tap_load_snapshot must have provided)."""
    return {
        H2TAP_Q14: {"order_line": ["ol_delivery_d", "ol_i_id", "ol_amount"],
                    "item": ["i_id", "i_data_p2"]},
        H2TAP_Q12: {"order_line": ["ol_w_id", "ol_d_id", "ol_o_id", "ol_delivery_d"],
                    "orders": ["o_w_id", "o_d_id", "o_id", "o_ol_cnt", "o_carrier_id", "o_entry_d"]},
        H2TAP_Q4: {"order_line": ["ol_w_id", "ol_d_id", "ol_o_id", "ol_delivery_d"],
                   "orders": ["o_w_id", "o_d_id", "o_id", "o_ol_cnt", "o_entry_d"]},
        H2TAP_Q3: {"order_line": ["ol_w_id", "ol_d_id", "ol_o_id", "ol_amount"],
                   "orders": ["o_w_id", "o_d_id", "o_id", "o_c_id", "o_ol_cnt", "o_entry_d"],
                   "customer": ["c_w_id", "c_d_id", "c_id", "c_state_p2"],
                   "new_order": ["no_w_id", "no_d_id", "no_o_id", "no_deleted"]},
        H2TAP_Q6: {"order_line": ["ol_delivery_d", "ol_quantity", "ol_amount"]},
        H2TAP_Q1: {"order_line": ["ol_number", "ol_delivery_d", "ol_quantity", "ol_amount"]},
        H2TAP_Q18: {"order_line": ["ol_w_id", "ol_d_id", "ol_o_id", "ol_amount"],
                    "orders": ["o_w_id", "o_d_id", "o_id", "o_c_id", "o_ol_cnt", "o_entry_d"],
                    "customer": ["c_w_id", "c_d_id", "c_id", "c_last"]},
    }


def hot_path_tables(tables: dict, plans=HOT_PATH_PLANS) -> dict:
    """The subset of generated columns that ``plans`` read (default: the hot path, Q1/Q6/Q18)."""
    want = {}
    spec_of = plan_columns()
    for spec in (spec_of[p] for p in plans):
        for t, cols in spec.items():
            want.setdefault(t, [])
            for c in cols:
                if c not in want[t]:
                    want[t].append(c)
    # optional columns (new_order.no_deleted: Delivery's tombstones) are taken when present
    return {t: {c: tables[t][c] for c in cols if c in tables[t] or (t, c) not in OPTIONAL_COLUMNS}
            for t, cols in want.items()}


OPTIONAL_COLUMNS = {("new_order", "no_deleted")}


def h2tap_layout_sum(engine: Engine, data, layout: int, nrows: int, ncols: int, columns, *,
                     col_stride: int = 0, pax_rows: int = 64):
    """NEXT-3 / NEXT-4: SELECT SUM(col_c1 + ... + col_cN) over an int32 table in ``layout``
    (H2TAP_DSM / H2TAP_PAX / H2TAP_NSM, §5.3). ``data``: a CUDA int32 tensor (HBM) or a
    PINNED CPU int32 tensor (read zero-copy over PCIe); ``columns``: attribute indices.
    Returns (sum or None for no rows, kernel ms)."""
    if not (hasattr(data, "data_ptr") and hasattr(data, "is_cuda")):
        raise ValueError("data must be a torch tensor (CUDA, or pinned CPU)")
    if data.is_cuda:  # the library's stream is not ordered after torch's: data must be written
        import torch
        torch.cuda.current_stream(data.device).synchronize()
    mask = 0
    for c in columns:
        mask |= 1 << int(c)
    t = h2tap_layout_table(data.data_ptr() if nrows else None, layout, ncols, nrows, col_stride, pax_rows)
    out, isnull, ms = C.c_int64(), C.c_int32(), C.c_double()
    _check(_lib.h2tap_layout_sum(engine.handle, C.byref(t), mask, C.byref(out), C.byref(isnull), C.byref(ms)))
    return (None if isnull.value else out.value), ms.value


def pinned_tables(tables: dict, capacity: dict | None = None, pad_rows: int = 64) -> dict:
    """NEXT-4 helper: copy ``tables`` ({table: {column: array}}) into PINNED host torch tensors
    for H2TAP_LOAD_ZERO_COPY. Each column's storage holds ``capacity[table]`` rows (default: its
    length) plus ``pad_rows`` of readable slack; the returned tensors are views of the first n rows
    — ``t.untyped_storage()`` spans the whole capacity, so later appends write rows in place and
    publish them with ``first_row`` (see tests/test_gpu_zero_copy.py)."""
    import torch
    out = {}
    for tname, cols in tables.items():
        out[tname] = {}
        for cname, a in cols.items():
            arr = np.ascontiguousarray(a)
            cap = max(len(arr), (capacity or {}).get(tname, 0))
            buf = torch.empty(cap + pad_rows, dtype=getattr(torch, arr.dtype.name), pin_memory=True)
            buf[:len(arr)].copy_(torch.from_numpy(arr))
            out[tname][cname] = buf[:len(arr)]
    return out
