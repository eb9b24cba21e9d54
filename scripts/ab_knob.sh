# quick knob sweep of the ORDER BY bucket size (bench only)
for d in -1 0 1; do
  H2TAP_BUCKET_BITS_DELTA=$d timeout 300 python bench.py --no-cpu-baseline --steps 10 2>&1 | tail -1 > gpurun_out/knob_$d.json
  python -c "
import json; d=json.load(open('gpurun_out/knob_$d.json'))
print('$d', d['ms_per_step'], {k: v['ms'] for k, v in d['kernels'].items() if 'sort' in k or 'bucket' in k})"
done
timeout 600 python -m pytest tests/test_gpu_parity.py -q -x --timeout 300 2>&1 | tail -2
