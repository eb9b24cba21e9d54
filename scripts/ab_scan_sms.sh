#!/bin/bash
for n in 148 111 96 74; do
  echo "== SCAN_SMS=$n"
  H2TAP_SCAN_SMS=$n timeout 600 python bench.py --steps 10 --warmup 3 --no-cpu-baseline --no-c1 2>/dev/null | tail -1 | python -c "
import json,sys
d=json.loads(sys.stdin.read())
print('step', round(d['ms_per_step'],4), 'q6_alone', d['latency_ms']['q6_alone'], 'q1_alone', d['latency_ms']['q1_alone'], 'shared', d['kernels']['q61_shared_scan']['ms'])
"
done
