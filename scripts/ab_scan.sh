# A/B of the scan kernel variants: full GPU tests with the defaults, then the probe variant and
# LDG-only runs of bench.py; ncu time of Q6 for both implementations.
mkdir -p gpurun_out
timeout 900 python -m pytest tests -m gpu -q --timeout 400 -rf -x 2>&1 | tail -3 | tee gpurun_out/pytest_gpu.txt
H2TAP_SCAN=ldg H2TAP_PROBE=tma timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -q --timeout 400 -x -k "parity_small or ragged or w100_bench" 2>&1 | tail -2 | tee -a gpurun_out/pytest_gpu.txt
timeout 600 python bench.py --steps 20 --warmup 5 --no-cpu-baseline 2>&1 | tail -1 > gpurun_out/bench_tma.txt
H2TAP_SCAN=ldg timeout 600 python bench.py --steps 20 --warmup 5 --no-cpu-baseline 2>&1 | tail -1 > gpurun_out/bench_ldg.txt
