#!/bin/bash
# A/B of Q18 knobs on the bench (kernel table of the instrumented pass)
mkdir -p gpurun_out
for cfg in "$@"; do
  echo "== $cfg"
  env $cfg timeout 600 python bench.py --steps 10 --warmup 3 --no-cpu-baseline --no-c1 2>/dev/null | tail -1 | python -c "
import json,sys
d=json.loads(sys.stdin.read())
print('step', round(d['ms_per_step'],4), 'q18', d['latency_ms']['q18_in_batch'])
for k,v in d['kernels'].items():
    if k.startswith('q18'): print('  ', k, v['ms'])
"
done
