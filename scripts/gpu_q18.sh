# Q18 ORDER BY iteration: Q18 parity tests, then the bench with carry on / off
mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_parity.py tests/test_gpu_q3.py -q -x --timeout 300 2>&1 | tail -3 | tee gpurun_out/pytest_q18.txt
for c in 1 0; do
  H2TAP_ORDER_CARRY=$c timeout 300 python bench.py --no-cpu-baseline --steps 10 2>&1 | tail -1 > gpurun_out/carry_$c.json
  python -c "
import json; d=json.load(open('gpurun_out/carry_$c.json'))
print('carry=$c', d['ms_per_step'], {k: v['ms'] for k, v in d['kernels'].items() if 'q18' in k})"
done
