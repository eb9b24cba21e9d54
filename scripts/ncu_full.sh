# one ncu --set full capture of the batch's full pass (Q6 + Q1 + Q18 probe), source-level stalls
mkdir -p gpurun_out
TAG=${1:-full}
ncu --set full --clock-control none --import-source on -k regex:'q1_tma_kernel' -c 1 \
    -o gpurun_out/prof_$TAG -f python scripts/profile_run.py --warehouses 100 --reps 1 > gpurun_out/prof_$TAG.log 2>&1
python scripts/ncu_lines.py gpurun_out/prof_$TAG.ncu-rep q1_tma_kernel 45 > gpurun_out/lines_$TAG.txt 2>&1
ncu -i gpurun_out/prof_$TAG.ncu-rep --page details --csv > gpurun_out/details_$TAG.csv 2>&1
tail -3 gpurun_out/prof_$TAG.log
