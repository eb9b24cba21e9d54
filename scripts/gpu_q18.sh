# Q18 iteration: Q18 parity tests (both ORDER BY front ends), then the bench A/B
mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_parity.py tests/test_gpu_q3.py tests/test_gpu_next2.py tests/test_gpu_updates.py -q -x --timeout 300 2>&1 | tail -3 | tee gpurun_out/pytest_q18.txt
H2TAP_ORDER=v1 timeout 600 python -m pytest tests/test_gpu_parity.py -q -x --timeout 300 -k "q18 or small" 2>&1 | tail -2
for v in default H2TAP_ORDER_CARRY=0 default; do
  env $([ $v = default ] || echo $v) timeout 300 python bench.py --no-cpu-baseline --steps 20 2>&1 | tail -1 > gpurun_out/ab_q18.json
  python -c "
import json; d=json.load(open('gpurun_out/ab_q18.json'))
print('$v', round(d['ms_per_step'],4), {k: v['ms'] for k, v in d['kernels'].items() if 'q18' in k})"
done
