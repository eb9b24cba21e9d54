#!/bin/bash
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_gpu_multirank.py -q -x 2>&1 | tail -2
bash scripts/ab_q18.sh H2TAP_KV_TOUCH=1
timeout 1500 python bench.py --total-warehouses 1000 --plans q18 --steps 5 --warmup 3 --e2e-steps 2 --no-c1 --no-cpu-baseline 2>/dev/null | tail -1 > gpurun_out/bench_q18_w1000.json
python -c "
import json; d=json.loads(open('gpurun_out/bench_q18_w1000.json').read())
print('W1000 q18 step', d['ms_per_step'])
for k,v in d['kernels'].items(): print('  ', k, v['ms'])"
