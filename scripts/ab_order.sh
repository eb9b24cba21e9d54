# A/B of the ORDER BY variants: Q18 parity (both variants) + bench step with per-kernel times.
mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_parity.py tests/test_gpu_q3.py -q -x --timeout 300 2>&1 | tail -15
H2TAP_ORDER=v1 timeout 600 python -m pytest tests/test_gpu_parity.py -q -x --timeout 300 -k "q18 or order or tie or sort" 2>&1 | tail -2
for v in v2 v1; do
  H2TAP_ORDER=$v timeout 300 python bench.py --no-cpu-baseline --steps 10 2>&1 | tail -1 > gpurun_out/ab_$v.json
  python -c "
import json; d=json.load(open('gpurun_out/ab_$v.json'))
print('$v', d['ms_per_step'], {k: v['ms'] for k, v in d['kernels'].items() if 'sort' in k or 'bucket' in k or 'plan' in k})"
done
