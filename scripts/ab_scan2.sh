mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_parity.py -q -x --timeout 300 -k "small or ragged or full_size_w100_bench or golden" 2>&1 | tail -2
for v in 1 2; do
  timeout 300 python bench.py --no-cpu-baseline --steps 20 2>&1 | tail -1 > gpurun_out/sc.json
  python -c "
import json; d=json.load(open('gpurun_out/sc.json'))
print('run$v', round(d['ms_per_step'],4), {k: (v['ms'], v.get('frac_hbm')) for k, v in d['kernels'].items() if k.startswith('q6') or k.startswith('q1_scan') or 'probe' in k})"
done
