mkdir -p gpurun_out
timeout 900 python -m pytest tests -m gpu -q --timeout 400 -rf -x 2>&1 | tail -5 | tee gpurun_out/pytest_gpu.txt
timeout 600 python scripts/htap_mixed.py --warehouses 100 --seconds 15 --epoch-ms 100 --out gpurun_out/htap_mixed.json 2>&1 | tail -5
