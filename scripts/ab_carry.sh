# carry-mode ORDER BY: bucket-size sweep + one ncu capture of the per-bucket sort/emit
mkdir -p gpurun_out
for d in -2 -1 0; do
  H2TAP_BUCKET_BITS_DELTA=$d timeout 300 python bench.py --no-cpu-baseline --steps 10 2>&1 | tail -1 > gpurun_out/knob_$d.json
  python -c "
import json; d=json.load(open('gpurun_out/knob_$d.json'))
print('$d', d['ms_per_step'], {k: v['ms'] for k, v in d['kernels'].items() if 'sort' in k or 'bucket' in k})"
done
ncu --set full --clock-control none --import-source on -k regex:'bucket_local_emit|ob_scatter|q18_having' -c 3 \
    -o gpurun_out/prof_emit -f python scripts/profile_run.py --warehouses 100 --reps 1 > gpurun_out/prof_emit.log 2>&1
