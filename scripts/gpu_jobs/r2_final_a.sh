#!/bin/bash
# Final round-2 evidence, part A: mixes (f2 paper-shape 4- and 8-mixes, c3
# pairs, c4 staggered 8-mix) and the isolated single-tenant overhead table.
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
timeout 900 python scripts/isolated.py --reps 8 bfs cutcp stencil tpacf histo spmv sgemm mriq sad lbm gridding histo_pipeline > gpurun_out/fa_isolated.log 2>&1
timeout 2400 python scripts/mixes.py --config f2 --repeat --k 4 --n 1000 --reps 2 --seed 2024 --out gpurun_out/fa_f2_k4.json > gpurun_out/fa_f2_k4.log 2>&1
timeout 1800 python scripts/mixes.py --config f2 --repeat --k 8 --n 500 --reps 2 --seed 2025 --out gpurun_out/fa_f2_k8.json > gpurun_out/fa_f2_k8.log 2>&1
timeout 900 python scripts/mixes.py --config c3 --reps 3 --out gpurun_out/fa_c3.json > gpurun_out/fa_c3.log 2>&1
timeout 600 python scripts/mixes.py --config c4 --reps 5 --out gpurun_out/fa_c4.json > gpurun_out/fa_c4.log 2>&1
