set -x
timeout 1200 python -m pytest tests -m gpu -x -q 2>&1 | tail -15
timeout 600 python scripts/isolated.py stencil histo bfs cutcp tpacf 2>&1 | tail -6
timeout 900 python bench.py --steps 5 --warmup 3 --out gpurun_out/bench_c2.json 2>&1 | tail -3
