"""Small Q18 runs for compute-sanitizer racecheck / memcheck (carry v3, v2 row path, dist loopback)."""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__)))))
import chgen
import paper_conf_cidr_appuswamykpa17_b200 as h
t = chgen.generate(1, 2, seed=1)
e = h.h2tap_open(0)
h.h2tap_load_snapshot(e, h.hot_path_tables(t), 1)
for having in (20000, 5_000_000):
    r = h.h2tap_run_query(e, h.H2TAP_Q18, [having]); print("Q18", having, r.nrows); r.free()
rs = h.h2tap_run_queries(e, [(6, None, 0), (1, None, 0), (18, None, 0)])
for r in rs: r.free()
h.h2tap_close(e)
print("done")
