# one full ncu capture of the Q18 per-bucket sort/emit (+ scatter, HAVING) for source-level stalls
mkdir -p gpurun_out
ncu --set full --clock-control none --import-source on -k regex:'bucket_local_emit|ob_scatter|q18_having' -c 3 \
    -o gpurun_out/prof_emit -f python scripts/profile_run.py --warehouses 100 --reps 1 > gpurun_out/prof_emit.log 2>&1
