#!/usr/bin/env python
"""Cost of the cross-GPU merges, measured on ONE GPU with N logical ranks.

N engines on cuda:0 (h2tap_peer_connect_local), W warehouses split over them, run the bench's
batch (Q6 + Q1 + Q18) from N host threads with per-kernel CUDA events (H2TAP_QUERY_PROFILE).
The ranks share one device, so the scans are N-way concurrent on one HBM and their times mean
nothing for N GPUs; what this measures is what a merge kernel itself costs — the push, the wait
(all ranks' flags), the fold — and the distributed ORDER BY's route / exchange kernels, with
the data moved through device memory instead of NVLink. Never a bench number.

With --empty every rank's tables are empty: the scans are trivial, every rank arrives at each
merge at about the same time, and the times are the merges' fixed cost (launch, pushes, flag
round trips, fold) on one device.

Usage: python scripts/loopback_bench.py [--warehouses 8] [--ranks 2,4,8] [--reps 5] [--empty] [--out F]
"""
import argparse
import json
import os
import sys

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import chgen  # noqa: E402
import paper_conf_cidr_appuswamykpa17_b200 as h  # noqa: E402

MERGE = ("q6_peer_allreduce", "q1_peer_push", "q1_peer_merge", "q18_dist_meta", "q18_dist_counts",
         "q18_dist_route", "q18_dist_send", "q18_dist_wait")


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--warehouses", type=int, default=8)
    ap.add_argument("--ranks", default="2,4,8")
    ap.add_argument("--reps", type=int, default=5)
    ap.add_argument("--empty", action="store_true")
    ap.add_argument("--out", default=None)
    a = ap.parse_args()
    out = {"how": __doc__.split("\n\n")[1].replace("\n", " "), "warehouses_total": 0 if a.empty else a.warehouses,
           "empty": a.empty, "runs": []}
    for n in [int(x) for x in a.ranks.split(",")]:
        parts = [chgen.generate(lo, lo if a.empty else hi, seed=1) for lo, hi in chgen.warehouse_ranges(a.warehouses, n)]
        engines = h.open_local_group(n, 0, 256 << 20)
        try:
            for e, t in zip(engines, parts):
                h.h2tap_load_snapshot(e, h.hot_path_tables(t), 1)
            q = [(h.H2TAP_Q6, None, h.H2TAP_RESULT_DEVICE | h.H2TAP_QUERY_PROFILE),
                 (h.H2TAP_Q1, None, h.H2TAP_RESULT_DEVICE | h.H2TAP_QUERY_PROFILE),
                 (h.H2TAP_Q18, None, h.H2TAP_RESULT_DEVICE | h.H2TAP_QUERY_PROFILE)]

            def run(e):
                rs = h.h2tap_run_queries(e, q)
                ks = [k for r in rs for k in r.kernels]
                for r in rs:
                    h.h2tap_free(r)
                return ks
            for _ in range(2):
                h.run_collective(engines, run)
            per = {}
            for _ in range(a.reps):
                for ks in h.run_collective(engines, run):
                    for name, ms in ks:
                        if name in MERGE:
                            per.setdefault(name, []).append(ms * 1e3)
            row = {"ranks": n, "merge_kernel_us_median": {k: round(float(np.median(v)), 2) for k, v in per.items()},
                   "merge_kernel_us_max": {k: round(float(np.max(v)), 2) for k, v in per.items()}}
            out["runs"].append(row)
            print(json.dumps(row), flush=True)
        finally:
            for e in engines:
                h.h2tap_close(e)
    if a.out:
        json.dump(out, open(a.out, "w"), indent=1)


if __name__ == "__main__":
    main()
