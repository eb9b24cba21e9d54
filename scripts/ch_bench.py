#!/usr/bin/env python
"""NEXT-2 measurement: CH Q14 / Q12 / Q4 / Q3 on one B200 at the bench workload (W=100, ~30 M
order_line rows, 'spread', seed 1), CH default parameters, snapshot resident in HBM.

Per query: K timed runs (CUDA events on the engine stream around the query; L2 flushed between
runs by writing 512 MB), then one instrumented run (H2TAP_QUERY_PROFILE) for per-kernel times.
Algorithmic bytes per kernel:
  q14_scan_join_sum : 20 B x n_ol (delivery 8, i_id 4, amount 8); the item map is on chip
  q12/q4 build      : 12 B x n_o read + 4 B x n_o slot written (+ 4 B x key box cleared)
  q12_probe_groupby : 20 B x n_ol (w, d, o, delivery) + 20 B x n_o (slot 4, entry 8, carrier 4, cnt 4)
  q4_semijoin_mark  : 20 B x n_ol + 13 B x n_o (slot 4, entry 8, mark 1)
  q4_count          : 5 B x n_o (mark 1, o_ol_cnt 4)
  q3_build          : 12 B x (n_o + n_c) read + 4 B x (n_o + n_c) slots + 16 B x n_o accumulators zeroed
  q3_mark           : 12 B x n_no read + 4 B orders slot + 8 B o_entry_d per new_order row
  q3_probe_groupjoin: 20 B x n_ol (w, d, o, amount) + 8 B x n_o (orders slot + multiplicity per run)
Parity of the same queries at this size: tests/test_gpu_next2.py::test_full_size_w100.

Usage: python scripts/ch_bench.py [--steps 20] [--warmup 3] [--out FILE]
"""
import argparse
import json
import os
import sys

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import chgen  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--warehouses", type=int, default=100)
    ap.add_argument("--steps", type=int, default=20)
    ap.add_argument("--warmup", type=int, default=3)
    ap.add_argument("--out", default=None)
    a = ap.parse_args()
    import torch
    import paper_conf_cidr_appuswamykpa17_b200 as h
    t = chgen.generate(1, a.warehouses + 1, seed=1)
    plans_all = (h.H2TAP_Q14, h.H2TAP_Q12, h.H2TAP_Q4, h.H2TAP_Q3)
    e = h.h2tap_open(0)
    h.h2tap_load_snapshot(e, h.hot_path_tables(t, plans_all), 1)
    n_ol, n_o = len(t["order_line"]["ol_o_id"]), len(t["orders"]["o_id"])
    n_c, n_no = len(t["customer"]["c_id"]), len(t["new_order"]["no_o_id"])
    peak = json.load(open(os.path.join(ROOT, "MEASURED_PEAKS.json")))["hbm_gbs"] \
        if os.path.exists(os.path.join(ROOT, "MEASURED_PEAKS.json")) else 6650.0
    alg = {"q14_scan_join_sum": 20 * n_ol, "q12_build": 16 * n_o, "q4_build": 16 * n_o,
           "q12_probe_groupby": 20 * n_ol + 20 * n_o, "q4_semijoin_mark": 20 * n_ol + 13 * n_o,
           "q4_count": 5 * n_o, "q3_build": 16 * (n_o + n_c) + 16 * n_o, "q3_mark": 24 * n_no,
           "q3_probe_groupjoin": 20 * n_ol + 8 * n_o}
    stream = torch.cuda.ExternalStream(h.h2tap_compute_stream(e))
    flush = torch.empty(512 << 20, dtype=torch.uint8, device="cuda")
    out = {}
    for name, plan in (("q14", h.H2TAP_Q14), ("q12", h.H2TAP_Q12), ("q4", h.H2TAP_Q4), ("q3", h.H2TAP_Q3)):
        ms = []
        for i in range(a.warmup + a.steps):
            flush.fill_(i & 0xff)
            torch.cuda.synchronize()
            with torch.cuda.stream(stream):
                b, en = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                b.record(stream)
                r = h.h2tap_run_query(e, plan, None, flags=h.H2TAP_RESULT_DEVICE)
                en.record(stream)
            torch.cuda.synchronize()
            h.h2tap_free(r)
            if i >= a.warmup:
                ms.append(b.elapsed_time(en))
        kern = {}
        for i in range(3):
            flush.fill_(7)
            torch.cuda.synchronize()
            r = h.h2tap_run_query(e, plan, None, flags=h.H2TAP_QUERY_PROFILE | h.H2TAP_RESULT_DEVICE)
            for k, v in r.kernels:
                kern.setdefault(k, []).append(v)
            flags, nrows = r.plan_flags, r.nrows
            h.h2tap_free(r)
        kstats = {}
        for k, v in kern.items():
            m = float(np.median(v))
            d = {"ms": round(m, 4)}
            if k in alg:
                d["alg_bytes"] = alg[k]
                d["GBps"] = round(alg[k] / (m * 1e-3) / 1e9, 1)
                d["frac_of_peak"] = round(alg[k] / (m * 1e-3) / 1e9 / peak, 3)
            kstats[k] = d
        out[name] = {"ms_median": round(float(np.median(ms)), 4), "ms_min": round(float(np.min(ms)), 4),
                     "order_line_rows_per_s": n_ol / (float(np.median(ms)) * 1e-3),
                     "plan_flags": flags, "result_rows": nrows, "kernels": kstats}
    h.h2tap_close(e)
    line = json.dumps({"what": "NEXT-2 CH Q14/Q12/Q4/Q3, one B200, snapshot resident, L2 flushed per run",
                       "warehouses": a.warehouses, "order_line_rows": n_ol, "orders_rows": n_o,
                       "customer_rows": n_c, "new_order_rows": n_no,
                       "peak_GBps": peak, "steps": a.steps, "queries": out})
    print(line)
    if a.out:
        open(a.out, "w").write(line + "\n")


if __name__ == "__main__":
    main()
