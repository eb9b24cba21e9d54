mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_parity.py -q --timeout 400 -x 2>&1 | tail -2
for v in 1 0 1; do
  H2TAP_SHARED_SCAN=$v timeout 300 python bench.py --no-cpu-baseline --steps 20 2>&1 | tail -1 > gpurun_out/ss.json
  python -c "
import json; d=json.load(open('gpurun_out/ss.json'))
print('shared=$v', round(d['ms_per_step'],4), d['latency_ms'], d['roofline']['kernel'], d['roofline']['frac'], {k: v['ms'] for k, v in d['kernels'].items() if k.startswith('q6') or k.startswith('q1_scan') or k.startswith('q61')})"
done
