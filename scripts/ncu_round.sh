# ncu evidence for one round: launch list (cold, serialised) + one full capture of every hot kernel.
# usage: bash scripts/ncu_round.sh <tag>
set -x
TAG=${1:-r01}
mkdir -p gpurun_out
ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_${TAG}.csv \
    python scripts/profile_run.py --warehouses 100 --reps 2 > gpurun_out/launches_${TAG}.log 2>&1
ncu --set full --clock-control none --import-source on \
    -k regex:'q6_tma_kernel|q1_tma_kernel|q18_|bucket_|ob_|l2_touch' \
    -c 30 -o gpurun_out/prof_${TAG} -f \
    python scripts/profile_run.py --warehouses 100 --reps 1 > gpurun_out/prof_${TAG}.log 2>&1
