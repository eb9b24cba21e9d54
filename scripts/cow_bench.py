#!/usr/bin/env python
"""NEXT-1 measurement: cost of an epoch of TPC-C Delivery updates on the W=100 snapshot
(30M order_line rows), page-granular copy-on-write vs whole-column copy (H2TAP_COW=full).

Per epoch size D (Delivery transactions per epoch; each delivers one order in each of the 10
districts of a warehouse, ~100 order_line rows + 10 orders rows), R refreshes of updates only
(h2tap_refresh, synchronous, update arrays in pinned host memory), reporting the copy-stream
CUDA-event times of the update phase (h2tap_store_stats): last_update_h2d_ms (row ids + values
over PCIe) and last_update_ms (device: shadow catch-up + scatter), the pages copied into
shadows, and the algorithmic bytes of the device work:
  catch-up: pages x 4096 rows x elem_size x 2 (read + write)
  scatter : n x (4 B row id + elem_size value) read + n x 32 B sector written
Parity of the same workload against the oracle is tests/test_gpu_updates.py (W=100 included).

Usage: python scripts/cow_bench.py [--warehouses 100] [--reps 10] [--out FILE]
  (run twice: once as is, once with H2TAP_COW=full; or --both to spawn the second run)
"""
import argparse
import json
import os
import subprocess
import sys
import time

import numpy as np
import torch

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import chgen  # noqa: E402
import paper_conf_cidr_appuswamykpa17_b200 as h  # noqa: E402

PAGE = 4096


def run(W, reps, sizes):
    t = chgen.generate(1, W + 1, seed=1)
    t.pop("item")
    hot = h.hot_path_tables(t)
    hot["orders"]["o_carrier_id"] = t["orders"]["o_carrier_id"]  # Delivery sets it too
    e = h.h2tap_open(0)
    st = chgen.DeliveryState()
    st.add(t["orders"], 0, 0)
    epoch = 1
    h.h2tap_load_snapshot(e, hot, epoch)
    clock = chgen.TS_2025 + chgen.DAY_US
    out = []
    b = 0
    for D in sizes:
        ms, h2d, pages, n_ol, n_o, full = [], [], [], [], [], []
        for r in range(reps + 1):  # first refresh of each size is a warm-up
            w, carrier = chgen.delivery_inputs(D, seed=1, batch=b, w_lo=1, w_hi=W + 1)
            b += 1
            upd = chgen.delivery_batch(st, w, carrier, clock)
            pinned = {tb: {c: (torch.from_numpy(r).pin_memory() if len(r) else r,
                               torch.from_numpy(v).pin_memory() if len(v) else v)
                           for c, (r, v) in per.items()} for tb, per in upd.items()}
            clock += (D + 1) * 1000
            s0 = h.h2tap_get_store_stats(e)
            epoch += 1
            h.h2tap_refresh(e, None, pinned, epoch)
            s1 = h.h2tap_get_store_stats(e)
            if r == 0:
                continue
            ms.append(s1["last_update_ms"])
            h2d.append(s1["last_update_h2d_ms"])
            pages.append(s1["cow_pages_copied"] - s0["cow_pages_copied"])
            full.append(s1["cow_full_copies"] - s0["cow_full_copies"])
            n_ol.append(len(upd["order_line"]["ol_delivery_d"][0]))
            n_o.append(len(upd["orders"]["o_carrier_id"][0]))
        nol, no = float(np.mean(n_ol)), float(np.mean(n_o))
        pg = float(np.mean(pages))
        # catch-up bytes: the page list mixes the 8 B ol_delivery_d pages and 4 B o_carrier_id
        # pages; bound it with the larger element size per page (conservative for GB/s)
        alg = pg * PAGE * 8 * 2 + nol * (4 + 8 + 32) + no * (4 + 4 + 32)
        out.append({"deliveries_per_epoch": D, "ol_rows_updated": nol, "orders_rows_updated": no,
                    "update_ms_median": float(np.median(ms)), "update_ms_min": float(np.min(ms)),
                    "update_h2d_ms_median": float(np.median(h2d)),
                    "device_GBps": alg / (float(np.median(ms)) * 1e-3) / 1e9,
                    "pages_copied": pg, "full_column_copies": float(np.mean(full)),
                    "alg_bytes": alg})
    res = {}
    h.h2tap_close(e)
    return out, res


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--warehouses", type=int, default=100)
    ap.add_argument("--reps", type=int, default=10)
    ap.add_argument("--sizes", default="10,100,1000,5000")
    ap.add_argument("--both", action="store_true", help="also run the H2TAP_COW=full baseline")
    ap.add_argument("--out", default=None)
    a = ap.parse_args()
    sizes = [int(x) for x in a.sizes.split(",")]
    mode = "full" if os.environ.get("H2TAP_COW") == "full" else "pages"
    t0 = time.time()
    rows, parity = run(a.warehouses, a.reps, sizes)
    line = {"what": "NEXT-1 Delivery update epochs, copy-stream device time per epoch",
            "cow": mode, "warehouses": a.warehouses, "order_line_rows": a.warehouses * 300_000,
            "results": rows, **parity, "wall_s": round(time.time() - t0, 1)}
    if a.both:
        env = dict(os.environ, H2TAP_COW="full")
        cmd = [sys.executable, __file__, "--warehouses", str(a.warehouses), "--reps", str(a.reps),
               "--sizes", a.sizes]
        base = json.loads(subprocess.check_output(cmd, env=env, text=True).strip().splitlines()[-1])
        line["baseline_full_copy"] = base["results"]
        for r, bsl in zip(rows, base["results"]):
            r["speedup_vs_full_copy"] = bsl["update_ms_median"] / r["update_ms_median"]
    s = json.dumps(line)
    print(s)
    if a.out:
        with open(a.out, "w") as f:
            f.write(s + "\n")


if __name__ == "__main__":
    main()
