python - <<'PY'
import sys, os, json
sys.path.insert(0, os.getcwd())
import chgen, torch
import paper_conf_cidr_appuswamykpa17_b200 as h
t = chgen.generate(1, 101, seed=1, mode="spread")
e = h.h2tap_open(0)
h.h2tap_load_snapshot(e, h.hot_path_tables(t), 1)
for thr in (20000, 20000):
    ks = {}
    for rep in range(8):
        r = h.h2tap_run_query(e, 18, [thr], flags=h.H2TAP_RESULT_DEVICE | h.H2TAP_QUERY_PROFILE)
        for k, ms in r.kernels:
            ks.setdefault(k, []).append(ms)
        h.h2tap_free(r)
    print(thr, {k: round(sorted(v)[len(v)//2] * 1e3, 1) for k, v in ks.items() if 'having' in k})
PY
