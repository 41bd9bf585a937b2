#!/bin/bash
# round 2 batch b: bench, weight rules, isolated overheads, sampled 4-mixes
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
timeout 300 python bench.py --steps 10 --warmup 3 > gpurun_out/r2b_bench.log 2>&1
timeout 600 python scripts/weights.py --reps 5 --grid 3 --out gpurun_out/r2b_weights.json > gpurun_out/r2b_weights.log 2>&1
timeout 600 python scripts/isolated.py --reps 10 bfs cutcp stencil tpacf histo spmv sgemm mriq > gpurun_out/r2b_isolated.log 2>&1
timeout 900 python scripts/mixes.py --config f2 --k 4 --n 100 --reps 2 --modes resolve,static --out gpurun_out/r2b_f2.json > gpurun_out/r2b_f2.log 2>&1
tail -c 600 gpurun_out/r2b_bench.log; tail -20 gpurun_out/r2b_weights.log; cat gpurun_out/r2b_isolated.log | cut -c 1-300; tail -2 gpurun_out/r2b_f2.log | cut -c 1-1500
