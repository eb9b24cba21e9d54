# PDL A/B: full GPU tests with PDL, then the bench with and without
mkdir -p gpurun_out
timeout 900 python -m pytest tests -m gpu -q --timeout 400 -x 2>&1 | tail -3 | tee gpurun_out/pytest_gpu.txt
for v in 1 0 1; do
  H2TAP_PDL=$v timeout 300 python bench.py --no-cpu-baseline --steps 20 2>&1 | tail -1 > gpurun_out/pdl.json
  python -c "
import json; d=json.load(open('gpurun_out/pdl.json'))
print('pdl=$v', round(d['ms_per_step'],4), round(sum(v['ms'] for v in d['kernels'].values()),4))"
done
