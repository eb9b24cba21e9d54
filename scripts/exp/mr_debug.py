"""Loopback debugging: 2 logical ranks on one GPU, one plan at a time."""
import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__)))))
os.environ.setdefault("H2TAP_PEER_TIMEOUT_MS", "3000")
import chgen
import paper_conf_cidr_appuswamykpa17_b200 as h

world = int(sys.argv[1]) if len(sys.argv) > 1 else 2
parts = [chgen.generate(lo, hi, seed=3) for lo, hi in chgen.warehouse_ranges(world + 1, world)]
for plans in ([h.H2TAP_Q6], [h.H2TAP_Q1], [h.H2TAP_Q18], [h.H2TAP_Q6, h.H2TAP_Q1, h.H2TAP_Q18]):
    engines = h.open_local_group(world, 0, 64 << 20)
    for e, t in zip(engines, parts):
        h.h2tap_load_snapshot(e, h.hot_path_tables(t), 1)
    t0 = time.time()
    try:
        out = h.run_collective(engines, lambda e: [(r.nrows, r.row_offset, r.total_rows) for r in h.h2tap_run_queries(e, [(p, None, 0) for p in plans])])
        print(plans, "OK", out, f"{time.time()-t0:.2f}s", flush=True)
    except Exception as x:
        print(plans, "FAIL", x, f"{time.time()-t0:.2f}s", flush=True)
    for e in engines:
        h.h2tap_close(e)
