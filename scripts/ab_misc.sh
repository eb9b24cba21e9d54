# A/B: HAVING unroll 2 vs 4 (bench kernel times); zero-copy scans LDG vs TMA (zero_copy_bench)
mkdir -p gpurun_out
for u in 2 4; do
  H2TAP_HAVING_UNROLL=$u timeout 300 python bench.py --no-cpu-baseline --steps 10 2>&1 | tail -1 > gpurun_out/hu_$u.json
  python -c "
import json; d=json.load(open('gpurun_out/hu_$u.json'))
print('having_unroll $u', d['ms_per_step'], d['kernels']['q18_having_compact'])"
done
H2TAP_HAVING_UNROLL=4 timeout 600 python -m pytest tests/test_gpu_parity.py -q -x --timeout 300 -k "q18" 2>&1 | tail -1
timeout 300 python scripts/zero_copy_bench.py --steps 5 --epochs 5 2>&1 | grep zero_copy | cut -c1-300
H2TAP_ZC_TMA=1 timeout 300 python scripts/zero_copy_bench.py --steps 5 --epochs 5 2>&1 | grep zero_copy | cut -c1-300
H2TAP_ZC_TMA=1 timeout 300 python -m pytest tests/test_gpu_zero_copy.py -q -x 2>&1 | tail -1
