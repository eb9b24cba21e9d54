set -x
TAG=${1:-q18}
mkdir -p gpurun_out
ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_${TAG}.csv \
    python scripts/profile_run.py --warehouses 100 --reps 2 --plans 18 > gpurun_out/launches_${TAG}.log 2>&1
ncu --set full --clock-control none --import-source on \
    -k regex:'q18_having|bucket_|q18_probe|q18_keys' -c 8 -o gpurun_out/prof_${TAG} -f \
    python scripts/profile_run.py --warehouses 100 --reps 1 --plans 18 > gpurun_out/prof_${TAG}.log 2>&1
