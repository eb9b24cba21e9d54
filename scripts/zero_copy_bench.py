#!/usr/bin/env python
"""NEXT-4 measurement: zero-copy host-resident snapshot (H2TAP_LOAD_ZERO_COPY: kernels read the
caller's pinned host columns over PCIe — Caldera's UVA mechanism)
versus the HBM snapshot refreshed by H2D copies (the north_star design), on one B200, W=100.

Reported per residency:
  * query latency (CUDA events on the engine stream, median of K) of Q6, Q1, Q18 and the scan's
    algorithmic GB/s (Q6 20 B/row, Q1 24 B/row) against the HBM copy peak or the pinned H2D
    bandwidth measured in the same run;
  * freshness: NewOrder batches of B transactions appended per epoch — wall time of the publish
    call (zero-copy: no copy, only the zone map of the new rows; HBM: H2D of the delta) and of
    publish + a Q6 on the new epoch ("time to a fresh result").

Usage: python scripts/zero_copy_bench.py [--warehouses 100] [--steps 10] [--batch 1000] [--out F]
"""
import argparse
import json
import os
import sys
import time

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import chgen  # noqa: E402

Q6_P = [chgen.ts_us("1999-01-01"), chgen.ts_us("2020-01-01"), 1, 100000]
Q1_P = [chgen.ts_us("2007-01-02")]


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--warehouses", type=int, default=100)
    ap.add_argument("--steps", type=int, default=10)
    ap.add_argument("--batch", type=int, default=1000, help="NewOrder transactions per epoch")
    ap.add_argument("--epochs", type=int, default=20)
    ap.add_argument("--out", default=None)
    a = ap.parse_args()
    import torch
    import paper_conf_cidr_appuswamykpa17_b200 as h
    W = a.warehouses
    t = chgen.generate(1, W + 1, seed=1)
    plans = (h.H2TAP_Q1, h.H2TAP_Q6, h.H2TAP_Q18)
    hot = h.hot_path_tables(t, plans)
    n_ol = len(t["order_line"]["ol_o_id"])
    st = chgen.NewOrderState(1, W + 1)
    deltas = [h.hot_path_tables({**chgen.neworder_batch(st, a.batch, seed=1, batch=b, item=t["item"]),
                                 "customer": t["customer"]}, plans) for b in range(a.epochs)]
    for d in deltas:
        d.pop("customer")
    extra = {k: sum(len(next(iter(d[k].values()))) for d in deltas) for k in ("order_line", "orders")}
    peaks = json.load(open(os.path.join(ROOT, "MEASURED_PEAKS.json"))) \
        if os.path.exists(os.path.join(ROOT, "MEASURED_PEAKS.json")) else {}
    hbm_peak = peaks.get("hbm_gbs", 6650.0)
    src = torch.empty(1 << 30, dtype=torch.uint8, pin_memory=True)
    dst = torch.empty(1 << 30, dtype=torch.uint8, device="cuda")
    ts = []
    for _ in range(5):
        b, en = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        b.record(); dst.copy_(src, non_blocking=True); en.record(); torch.cuda.synchronize()
        ts.append(b.elapsed_time(en))
    pcie = (1 << 30) / (np.median(ts[1:]) * 1e-3) / 1e9
    del src, dst
    out = {}
    for mode in ("hbm", "zero_copy"):
        e = h.h2tap_open(0)
        stream = torch.cuda.ExternalStream(h.h2tap_compute_stream(e))
        zc = mode == "zero_copy"
        cap = {k: len(next(iter(hot[k].values()))) + extra.get(k, 0) for k in hot}
        src_tabs = h.pinned_tables(hot, cap) if zc else hot
        flags = h.H2TAP_LOAD_ZERO_COPY if zc else 0
        h.h2tap_load_snapshot(e, src_tabs, 1, flags=flags)
        lat = {}
        for name, plan, p in (("q6", h.H2TAP_Q6, Q6_P), ("q1", h.H2TAP_Q1, Q1_P), ("q18", h.H2TAP_Q18, [20000])):
            ms = []
            for i in range(a.steps + 2):
                torch.cuda.synchronize()
                with torch.cuda.stream(stream):
                    b, en = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                    b.record(stream)
                    r = h.h2tap_run_query(e, plan, p, flags=h.H2TAP_RESULT_DEVICE)
                    en.record(stream)
                torch.cuda.synchronize()
                h.h2tap_free(r)
                if i >= 2:
                    ms.append(b.elapsed_time(en))
            lat[name] = round(float(np.median(ms)), 4)
        peak = pcie if zc else hbm_peak
        scan = {"q6_GBps": round(20 * n_ol / (lat["q6"] * 1e-3) / 1e9, 1),
                "q1_GBps": round(24 * n_ol / (lat["q1"] * 1e-3) / 1e9, 1)}
        scan["q6_frac"] = round(scan["q6_GBps"] / peak, 3)
        scan["q1_frac"] = round(scan["q1_GBps"] / peak, 3)
        # freshness: append epochs
        first = {k: len(next(iter(hot[k].values()))) for k in ("order_line", "orders")}
        pub, fresh = [], []
        for ep, d in enumerate(deltas):
            if zc:
                dt = {}
                for k, cols in d.items():
                    dt[k] = {}
                    for c, arr in cols.items():
                        full = src_tabs[k][c].as_strided((first[k] + len(arr),), (1,))
                        full[first[k]:].copy_(torch.from_numpy(np.ascontiguousarray(arr)))  # the OLTP write
                        dt[k][c] = full[first[k]:]
            else:
                dt = d
            t0 = time.perf_counter()
            h.h2tap_load_snapshot(e, dt, 2 + ep, flags=flags, full_reload=False, first_row=first)
            t1 = time.perf_counter()
            r = h.h2tap_run_query(e, h.H2TAP_Q6, Q6_P)
            t2 = time.perf_counter()
            assert r.epoch == 2 + ep
            h.h2tap_free(r)
            pub.append((t1 - t0) * 1e3)
            fresh.append((t2 - t0) * 1e3)
            for k in first:
                first[k] += len(next(iter(d[k].values())))
        out[mode] = {"latency_ms": lat, "scan": scan, "peak_GBps": round(peak, 1),
                     "publish_ms_p50": round(float(np.median(pub)), 4),
                     "publish_ms_p99": round(float(np.percentile(pub, 99)), 4),
                     "fresh_q6_ms_p50": round(float(np.median(fresh)), 4),
                     "device_bytes": h.h2tap_get_store_stats(e)["device_bytes"]}
        h.h2tap_close(e)
        print(json.dumps({mode: out[mode]}), flush=True)
    line = {"what": "NEXT-4 zero-copy host-resident vs HBM snapshot, one B200", "warehouses": W,
            "order_line_rows": n_ol, "neworder_per_epoch": a.batch, "epochs": a.epochs,
            "pcie_h2d_GBps": round(pcie, 1), "hbm_peak_GBps": hbm_peak, "modes": out}
    if a.out:
        open(a.out, "w").write(json.dumps(line) + "\n")


if __name__ == "__main__":
    main()
