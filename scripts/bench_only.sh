mkdir -p gpurun_out
timeout 600 python bench.py --steps 20 --warmup 5 --no-cpu-baseline "$@" 2>&1 | tail -3 | tee gpurun_out/bench.txt
