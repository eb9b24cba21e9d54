#!/bin/bash
# ncu captures of the Q18 v3 post-probe chain (launch list + --set full of each kernel once)
TAG=${1:-q18v3}
mkdir -p gpurun_out
ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_${TAG}.csv \
    python scripts/profile_run.py --warehouses 100 --reps 2 --plans 18 > gpurun_out/launches_${TAG}.log 2>&1
ncu --set full --clock-control none --import-source on \
    -k regex:'q18_acc_stats|q18_having_rec|ob_scatter_rec|bucket_local_emit|ob_scan|q18_build|q18_init' -c 8 \
    -o gpurun_out/prof_${TAG} -f \
    python scripts/profile_run.py --warehouses 100 --reps 1 --plans 18 > gpurun_out/prof_${TAG}.log 2>&1
echo ncu_done
