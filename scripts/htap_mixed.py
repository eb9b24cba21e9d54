#!/usr/bin/env python
"""Config C5 (BASELINE.json configs[4]) on one GPU: mixed HTAP run.

Three activities run concurrently (SURVEY.md §3 "mixed HTAP"):
  * OLTP: host threads run TPC-C NewOrder transactions into a host NSM row store (numpy records)
    — the task-parallel archipelago's side (PAPER.md L587-630 is out of scope; this is a driver);
  * epoch cutter: every E ms the rows committed since the last cut are refreshed into the HBM
    snapshot with h2tap_load_snapshot_rows (NSM -> DSM column extraction + H2D on the copy
    stream) and published as a new epoch (the paper's snapshot-per-epoch, L555-572);
  * OLAP: the query loop runs Q6+Q1+Q18 batches on the latest published epoch.
Reported: NewOrder tx/s, refresh MB/s, query batches/s, freshness lag p50/p99 (query start minus
the cut time of the epoch it read), and a final parity check of the last epoch against the oracle.

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


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--warehouses", type=int, default=100)
    ap.add_argument("--seconds", type=float, default=20.0)
    ap.add_argument("--epoch-ms", type=float, default=100.0)
    ap.add_argument("--txn-batch", type=int, default=2000)
    ap.add_argument("--tps", type=float, default=200_000.0, help="NewOrder rate the driver offers")
    ap.add_argument("--no-verify", action="store_true")
    ap.add_argument("--out", default=None)
    a = ap.parse_args()
    sys.setswitchinterval(0.0002)  # three Python threads share the GIL: switch often

    W = a.warehouses
    t = chgen.generate(1, W + 1, seed=1)
    item = t.pop("item")
    hot = h.hot_path_tables(t)
    cols = {tb: list(c) for tb, c in hot.items()}
    max_txn = int(a.tps * (a.seconds + 5) * 1.2) + a.txn_batch
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
    stats = {"txns": 0, "refresh_bytes": 0, "refresh_s": 0.0, "refreshes": 0}
    errors = []
    st = chgen.NewOrderState(1, W + 1)

    def oltp():
        b = 0
        t_start = time.perf_counter()
        try:
            while not stop.is_set():
                # offered load: a.tps NewOrder transactions per second
                ahead = (b * a.txn_batch) / a.tps - (time.perf_counter() - t_start)
                if ahead > 0:
                    time.sleep(ahead)
                d = chgen.neworder_batch(st, a.txn_batch, seed=1, batch=b, item=item)
                b += 1
                with lock:  # commit: rows become visible to the next epoch cut
                    stores["orders"].append(d["orders"])
                    stores["order_line"].append(d["order_line"])
                    stats["txns"] += a.txn_batch
        except Exception as x:  # pragma: no cover
            errors.append(x)

    def cutter():
        try:
            while not stop.is_set():
                time.sleep(a.epoch_ms / 1e3)
                with lock:
                    n = {tb: stores[tb].n for tb in ("order_line", "orders")}
                    txns = stats["txns"]
                    t_cut = time.perf_counter()  # the new epoch's logical time
                delta = {tb: stores[tb].rec[loaded[tb]:n[tb]] for tb in n}
                cut_time[epoch[0] + 1] = t_cut
                cut_txns[epoch[0] + 1] = txns
                t0 = time.perf_counter()
                h.h2tap_load_snapshot_rows(e, delta, epoch[0] + 1, full_reload=False,
                                           first_row={tb: loaded[tb] for tb in n},
                                           columns=cols, flags=h.H2TAP_LOAD_ASYNC)
                h.h2tap_sync(e)
                t1 = time.perf_counter()
                epoch[0] += 1
                stats["refresh_bytes"] += sum(
                    (n[tb] - loaded[tb]) * sum(np.dtype(chgen.ROW_DTYPES[tb][c]).itemsize for c in cols[tb])
                    for tb in n)
                stats["refresh_s"] += t1 - t0
                stats["refreshes"] += 1
                for tb in n:
                    loaded[tb] = n[tb]
        except Exception as x:  # pragma: no cover
            errors.append(x)

    q6 = [chgen.ts_us("1999-01-01"), chgen.ts_us("2020-01-01"), 1, 100000]
    batch = [(h.H2TAP_Q6, q6, h.H2TAP_RESULT_DEVICE), (h.H2TAP_Q1, None, h.H2TAP_RESULT_DEVICE),
             (h.H2TAP_Q18, None, h.H2TAP_RESULT_DEVICE)]
    threads = [threading.Thread(target=oltp), threading.Thread(target=cutter)]
    t_begin = time.perf_counter()
    for th in threads:
        th.start()
    lags, stale_txns, lat, epochs_seen, nq = [], [], [], set(), 0
    while time.perf_counter() - t_begin < a.seconds:
        tq = time.perf_counter()
        with lock:
            txns_now = stats["txns"]
        rs = h.h2tap_run_queries(e, batch)
        t_done = time.perf_counter()
        ep = rs[0].epoch
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

    out = {
        "config": f"C5 mixed HTAP, W={W}, 1 GPU, epoch period {a.epoch_ms} ms, "
                  f"NewOrder offered at {a.tps:.0f} tx/s in batches of {a.txn_batch} (1 host thread)",
        "seconds": round(wall, 2),
        "neworder_tx_per_s": stats["txns"] / wall,
        "epochs_published": stats["refreshes"],
        "refresh_MB_per_s_while_refreshing": stats["refresh_bytes"] / max(stats["refresh_s"], 1e-9) / 1e6,
        "refresh_ms_per_epoch_mean": stats["refresh_s"] / max(stats["refreshes"], 1) * 1e3,
        "query_batches_per_s": nq / wall,
        "batch_latency_ms_p50": float(np.percentile(lat, 50)),
        "batch_latency_ms_p99": float(np.percentile(lat, 99)),
        "freshness_lag_ms_p50": float(np.percentile(lags, 50)),
        "freshness_lag_ms_p99": float(np.percentile(lags, 99)),
        "staleness_txns_p50": float(np.percentile(stale_txns, 50)),
        "distinct_epochs_read": len(epochs_seen),
        "final_order_line_rows": stores["order_line"].n,
    }
    if not a.no_verify:  # the last published epoch against the oracle over the row store
        import oracle
        h.h2tap_sync(e)
        final = {tb: {c: np.ascontiguousarray(stores[tb].rec[c][:loaded.get(tb, stores[tb].n)])
                      for c in stores[tb].rec.dtype.names} for tb in stores}
        r18 = h.h2tap_run_query(e, h.H2TAP_Q18, [-1])
        got = r18.to_numpy()
        h.h2tap_free(r18)
        want = oracle.q18(final, -1)
        out["final_epoch_q18_parity"] = all(np.array_equal(got[k], want[k]) for k in want)
        r6 = h.h2tap_run_query(e, h.H2TAP_Q6, q6)
        out["final_epoch_q6_parity"] = int(r6.to_numpy()["revenue"][0]) == oracle.q6(final, *q6)["revenue"]
        h.h2tap_free(r6)
    h.h2tap_close(e)
    line = json.dumps(out)
    print(line)
    if a.out:
        with open(a.out, "w") as f:
            f.write(line + "\n")


if __name__ == "__main__":
    main()
