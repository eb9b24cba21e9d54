"""Short driver for ncu captures: W warehouses resident, each plan run `reps` times.

Never a bench number (run under ncu). Usage:
  ncu --set full ... python scripts/profile_run.py --warehouses 100 --reps 2
"""
import argparse
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import chgen  # noqa: E402
import paper_conf_cidr_appuswamykpa17_b200 as h  # noqa: E402

ap = argparse.ArgumentParser()
ap.add_argument("--warehouses", type=int, default=100)
ap.add_argument("--reps", type=int, default=2)
ap.add_argument("--plans", default="6,1,18")
ap.add_argument("--flags", type=int, default=h.H2TAP_RESULT_DEVICE)
ap.add_argument("--single", action="store_true", help="one h2tap_run_query per plan instead of one "
                "batch per rep (the bench's step is a batch: shared Q6+Q1 scan)")
a = ap.parse_args()

t = chgen.generate(1, a.warehouses + 1, seed=1, mode="spread")
e = h.h2tap_open(0)
h.h2tap_load_snapshot(e, h.hot_path_tables(t), 1)
plans = [int(x) for x in a.plans.split(",")]
for _ in range(a.reps):
    if a.single:
        for p in plans:
            h.h2tap_free(h.h2tap_run_query(e, p, flags=a.flags))
    else:
        for r in h.h2tap_run_queries(e, [(p, None, a.flags) for p in plans]):
            h.h2tap_free(r)
h.h2tap_close(e)
print("done")
