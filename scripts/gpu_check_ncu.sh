mkdir -p gpurun_out
timeout 900 python -m pytest tests -m gpu -q --timeout 400 -rf -x 2>&1 | tail -5 | tee gpurun_out/pytest_gpu.txt
timeout 600 python bench.py --steps 10 --warmup 3 --no-cpu-baseline 2>&1 | tail -3 | tee gpurun_out/bench.txt
bash scripts/ncu_q18.sh ${1:-q18b}
