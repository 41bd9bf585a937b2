# re-entry verification: GPU parity suite, default bench line, single-tenant dispatch overhead
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
timeout 1200 python -m pytest tests -m gpu -q -x 2>&1 | tail -3
timeout 900 python bench.py --steps 10 --warmup 3 --out gpurun_out/bench_c2.json > gpurun_out/bench_c2.log 2>&1; tail -c 600 gpurun_out/bench_c2.log
timeout 600 python scripts/isolated.py stencil histo bfs spmv sgemm mriq cutcp tpacf --reps 3 > gpurun_out/isolated.log 2>&1; cut -c1-400 gpurun_out/isolated.log
