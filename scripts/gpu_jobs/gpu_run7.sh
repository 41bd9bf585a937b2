timeout 1500 python -m pytest tests -m gpu -q -x 2>&1 | tail -5
timeout 600 python scripts/isolated.py stencil histo bfs cutcp tpacf spmv sgemm mriq 2>&1 | tail -8
timeout 600 python scripts/isolated.py stencil histo spmv bfs --chunk 2 2>&1 | tail -4
timeout 900 python bench.py --steps 5 --warmup 3 --out gpurun_out/bench_c2_r3.json 2>&1 | tail -1 | cut -c1-1500
