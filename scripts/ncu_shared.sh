mkdir -p gpurun_out
ncu --set full --clock-control none --import-source on -k regex:'q1_tma_kernel' -c 2 \
    -o gpurun_out/prof_shared -f python scripts/profile_run.py --warehouses 100 --reps 1 > gpurun_out/prof_shared.log 2>&1
H2TAP_SHARED_SCAN=0 ncu --set full --clock-control none --import-source on -k regex:'q1_tma_kernel' -c 1 \
    -o gpurun_out/prof_q1only -f python scripts/profile_run.py --warehouses 100 --reps 1 > gpurun_out/prof_q1only.log 2>&1
