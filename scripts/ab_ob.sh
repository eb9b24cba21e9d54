mkdir -p gpurun_out
for v in 2 1 2 1; do
  H2TAP_OB_PER_SM=$v timeout 300 python bench.py --no-cpu-baseline --steps 20 2>&1 | tail -1 > gpurun_out/ob.json
  python -c "
import json; d=json.load(open('gpurun_out/ob.json'))
print('per_sm=$v', round(d['ms_per_step'],4), {k: v['ms'] for k, v in d['kernels'].items() if 'sort' in k or 'bucket' in k})"
done
