# carry sort: rows per sub-bucket sweep (H2TAP_SUB_ROWS_LOG2)
mkdir -p gpurun_out
for d in 1 2 3 4; do
  H2TAP_SUB_ROWS_LOG2=$d timeout 300 python bench.py --no-cpu-baseline --steps 10 2>&1 | tail -1 > gpurun_out/sub_$d.json
  python -c "
import json; d=json.load(open('gpurun_out/sub_$d.json'))
print('$d', d['ms_per_step'], {k: v['ms'] for k, v in d['kernels'].items() if 'sort' in k or 'bucket' in k})"
done
