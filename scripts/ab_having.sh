# HAVING grid (blocks per SM) x unroll sweep
mkdir -p gpurun_out
for u in 2 4; do for b in 4 8 32; do
  H2TAP_HAVING_UNROLL=$u H2TAP_HAVING_BPS=$b timeout 300 python bench.py --no-cpu-baseline --steps 10 2>&1 | tail -1 > gpurun_out/hv.json
  python -c "
import json; d=json.load(open('gpurun_out/hv.json'))
print('u=$u bps=$b', round(d['ms_per_step'],4), d['kernels']['q18_having_compact']['ms'])"
done; done
