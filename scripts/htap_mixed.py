#!/usr/bin/env python
"""Config C5 (BASELINE.json configs[4]) on one GPU: mixed HTAP run.

Three activities run concurrently (SURVEY.md §3 "mixed HTAP"):
  * OLTP: a host thread runs TPC-C NewOrder and Delivery transactions (TPC-C mix ratio 45:4 by
    default) against a host NSM row store (numpy records): NewOrder appends orders and lines,
    Delivery updates o_carrier_id and ol_delivery_d in place — the task-parallel archipelago's
    side (PAPER.md L587-630 is out of scope; this is a driver);
  * epoch cutter: every E ms the rows committed since the last cut and the row updates since the
    last cut are refreshed into the HBM snapshot with h2tap_refresh_rows (NSM -> DSM column
    extraction + H2D, then copy-on-write of the updated columns, on the copy stream) and
    published as a new epoch (the paper's snapshot-per-epoch, L555-572; CoW L573-586);
  * OLAP: the query loop runs Q6+Q1+Q18 batches on the latest published epoch.
Reported: NewOrder tx/s, refresh MB/s, query batches/s, freshness lag p50/p99 (query start minus
the cut time of the epoch it read). Deliveries make Q1/Q6 freshness-observable.
Parity of the final epoch against the oracle: tests/test_gpu_mixed.py runs ``run()`` small.

Usage: python scripts/htap_mixed.py [--warehouses 100] [--seconds 20] [--epoch-ms 100]
"""
import argparse
import json
import os
import sys
import threading
import time

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import chgen  # noqa: E402
import paper_conf_cidr_appuswamykpa17_b200 as h  # noqa: E402


class RowStore:
    """Append-only host NSM row store for one table (capacity-doubling numpy records)."""

    def __init__(self, table, records, extra):
        self.table = table
        self.rec = np.empty(len(records) + extra, chgen.ROW_DTYPES[table])
        self.rec[:len(records)] = records
        self.n = len(records)

    def append(self, cols):
        r = chgen.to_records(self.table, cols)
        if self.n + len(r) > len(self.rec):
            raise RuntimeError(f"{self.table} row store full")
        self.rec[self.n:self.n + len(r)] = r
        self.n += len(r)

    def update(self, column, rows, values):
        self.rec[column][rows] = values


def run(W=100, seconds=20.0, epoch_ms=100.0, txn_batch=2000, tps=200_000.0, delivery_ratio=4 / 45,
        on_final=None):
    """Run the mixed workload; returns the report dict. ``on_final(engine, tables)`` is called
    after the last cut is published with the final row store as column arrays (what the last
    epoch must equal)."""
    sys.setswitchinterval(0.0002)  # three Python threads share the GIL: switch often
    t = chgen.generate(1, W + 1, seed=1)
    item = t.pop("item")
    hot = h.hot_path_tables(t)
    cols = {tb: list(c) for tb, c in hot.items()}
    cols["orders"].append("o_carrier_id")  # Delivery sets it
    max_txn = int(tps * (seconds + 5) * 1.2) + txn_batch
    extra = {"order_line": 15 * max_txn, "orders": max_txn, "customer": 0}
    stores = {tb: RowStore(tb, chgen.to_records(tb, t[tb]), extra=extra[tb])
              for tb in ("order_line", "orders", "customer")}
    e = h.h2tap_open(0)
    lock = threading.Lock()
    epoch = [1]
    h.h2tap_load_snapshot_rows(e, {tb: s.rec[:s.n] for tb, s in stores.items()}, epoch[0], columns=cols)
    loaded = {tb: s.n for tb, s in stores.items()}
    for tb in ("order_line", "orders"):  # appends never reallocate on the refresh path
        h.h2tap_reserve(e, tb, len(stores[tb].rec))
    cut_time = {epoch[0]: time.perf_counter()}
    cut_txns = {epoch[0]: 0}
    stop = threading.Event()
    stats = {"txns": 0, "deliveries": 0, "refresh_bytes": 0, "refresh_s": 0.0, "refreshes": 0,
             "rows_updated": 0}
    errors = []
    st = chgen.NewOrderState(1, W + 1)
    dl = chgen.DeliveryState()
    dl.add(t["orders"], 0, 0)
    pending_upd = {("orders", "o_carrier_id"): [], ("order_line", "ol_delivery_d"): []}
    n_del = max(0, int(round(txn_batch * delivery_ratio)))

    def oltp():
        b = 0
        t_start = time.perf_counter()
        try:
            while not stop.is_set():
                # offered load: tps NewOrder transactions per second
                ahead = (b * txn_batch) / tps - (time.perf_counter() - t_start)
                if ahead > 0:
                    time.sleep(ahead)
                d = chgen.neworder_batch(st, txn_batch, seed=1, batch=b, item=item)
                w, carrier = chgen.delivery_inputs(n_del, seed=1, batch=b, w_lo=1, w_hi=W + 1)
                b += 1
                with lock:  # commit: rows and updates become visible to the next epoch cut
                    n_o, n_ol = stores["orders"].n, stores["order_line"].n
                    stores["orders"].append(d["orders"])
                    stores["order_line"].append(d["order_line"])
                    dl.add(d["orders"], n_o, n_ol)
                    upd = chgen.delivery_batch(dl, w, carrier, st.clock)
                    for tb, per_col in upd.items():
                        for c, (rows, vals) in per_col.items():
                            stores[tb].update(c, rows, vals)
                            pending_upd[(tb, c)].append((rows, vals))
                    stats["txns"] += txn_batch
                    stats["deliveries"] += n_del
        except Exception as x:  # pragma: no cover
            errors.append(x)

    def cut():
        with lock:
            n = {tb: stores[tb].n for tb in ("order_line", "orders")}
            txns = stats["txns"]
            t_cut = time.perf_counter()  # the new epoch's logical time
            delta = {tb: stores[tb].rec[loaded[tb]:n[tb]].copy() for tb in n}
            taken = {k: v for k, v in pending_upd.items()}
            for k in pending_upd:
                pending_upd[k] = []
        updates = {}
        for (tb, c), parts in taken.items():
            if parts:
                updates.setdefault(tb, {})[c] = (np.concatenate([p[0] for p in parts]),
                                                 np.concatenate([p[1] for p in parts]))
        cut_time[epoch[0] + 1] = t_cut
        cut_txns[epoch[0] + 1] = txns
        t0 = time.perf_counter()
        h.h2tap_refresh_rows(e, delta, updates, epoch[0] + 1,
                             first_row={tb: loaded[tb] for tb in n}, columns=cols,
                             flags=h.H2TAP_LOAD_ASYNC)
        h.h2tap_sync(e)
        t1 = time.perf_counter()
        epoch[0] += 1
        stats["refresh_bytes"] += sum(
            (n[tb] - loaded[tb]) * sum(np.dtype(chgen.ROW_DTYPES[tb][c]).itemsize for c in cols[tb])
            for tb in n) + sum(len(r) * (4 + v.itemsize) for per in updates.values() for r, v in per.values())
        stats["rows_updated"] += sum(len(r) for per in updates.values() for r, _ in per.values())
        stats["refresh_s"] += t1 - t0
        stats["refreshes"] += 1
        for tb in n:
            loaded[tb] = n[tb]

    def cutter():
        try:
            while not stop.is_set():
                time.sleep(epoch_ms / 1e3)
                cut()
        except Exception as x:  # pragma: no cover
            errors.append(x)

    q6 = [chgen.ts_us("1999-01-01"), chgen.ts_us("2020-01-01"), 1, 100000]
    q1_fresh = [chgen.TS_2025]  # counts exactly the lines delivered since the load
    batch = [(h.H2TAP_Q1, q1_fresh, 0), (h.H2TAP_Q6, q6, h.H2TAP_RESULT_DEVICE),
             (h.H2TAP_Q1, None, h.H2TAP_RESULT_DEVICE), (h.H2TAP_Q18, None, h.H2TAP_RESULT_DEVICE)]
    threads = [threading.Thread(target=oltp), threading.Thread(target=cutter)]
    t_begin = time.perf_counter()
    for th in threads:
        th.start()
    lags, stale_txns, lat, epochs_seen, nq = [], [], [], set(), 0
    delivered_seen = []
    while time.perf_counter() - t_begin < seconds:
        tq = time.perf_counter()
        with lock:
            txns_now = stats["txns"]
        rs = h.h2tap_run_queries(e, batch)
        t_done = time.perf_counter()
        ep = rs[0].epoch
        delivered_seen.append(int(rs[0].to_numpy()["count_order"].sum()))
        for r in rs:
            h.h2tap_free(r)
        nq += 1
        epochs_seen.add(ep)
        lags.append((tq - cut_time[ep]) * 1e3)
        stale_txns.append(txns_now - cut_txns[ep])
        lat.append((t_done - tq) * 1e3)
    stop.set()
    for th in threads:
        th.join()
    wall = time.perf_counter() - t_begin
    if errors:
        raise errors[0]
    cut()  # the final epoch holds every committed transaction
    ss = h.h2tap_get_store_stats(e)
    out = {
        "config": f"C5 mixed HTAP, W={W}, 1 GPU, epoch period {epoch_ms} ms, "
                  f"NewOrder offered at {tps:.0f} tx/s in batches of {txn_batch}, "
                  f"{n_del} Delivery per batch (1 host thread)",
        "seconds": round(wall, 2),
        "neworder_tx_per_s": stats["txns"] / wall,
        "delivery_tx_per_s": stats["deliveries"] / wall,
        "epochs_published": stats["refreshes"],
        "rows_updated": stats["rows_updated"],
        "refresh_MB_per_s_while_refreshing": stats["refresh_bytes"] / max(stats["refresh_s"], 1e-9) / 1e6,
        "refresh_ms_per_epoch_mean": stats["refresh_s"] / max(stats["refreshes"], 1) * 1e3,
        "cow_pages_copied": ss["cow_pages_copied"], "cow_full_copies": ss["cow_full_copies"],
        "query_batches_per_s": nq / wall,
        "batch_latency_ms_p50": float(np.percentile(lat, 50)),
        "batch_latency_ms_p99": float(np.percentile(lat, 99)),
        "freshness_lag_ms_p50": float(np.percentile(lags, 50)),
        "freshness_lag_ms_p99": float(np.percentile(lags, 99)),
        "staleness_txns_p50": float(np.percentile(stale_txns, 50)),
        "distinct_epochs_read": len(epochs_seen),
        "q1_delivered_lines_first_last": [delivered_seen[0], delivered_seen[-1]] if delivered_seen else None,
        "final_order_line_rows": stores["order_line"].n,
    }
    if on_final is not None:
        final = {tb: {c: np.ascontiguousarray(stores[tb].rec[c][:stores[tb].n])
                      for c in stores[tb].rec.dtype.names} for tb in stores}
        on_final(e, final)
    h.h2tap_close(e)
    return out


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--warehouses", type=int, default=100)
    ap.add_argument("--seconds", type=float, default=20.0)
    ap.add_argument("--epoch-ms", type=float, default=100.0)
    ap.add_argument("--txn-batch", type=int, default=2000)
    ap.add_argument("--tps", type=float, default=200_000.0, help="NewOrder rate the driver offers")
    ap.add_argument("--delivery-ratio", type=float, default=4 / 45,
                    help="Delivery transactions per NewOrder (TPC-C mix 4%%:45%%)")
    ap.add_argument("--out", default=None)
    a = ap.parse_args()
    out = run(a.warehouses, a.seconds, a.epoch_ms, a.txn_batch, a.tps, a.delivery_ratio)
    line = json.dumps(out)
    print(line)
    if a.out:
        with open(a.out, "w") as f:
            f.write(line + "\n")


if __name__ == "__main__":
    main()
