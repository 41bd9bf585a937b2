#!/bin/bash
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
for h in 1 2; do echo "== l2hint $h"; ACCEL_TMA_L2HINT=$h timeout 600 python scripts/diag_tma.py --reps 2 --sweeps 40 --combos=-,bfs 2>&1; done | tee gpurun_out/r2t_diag_hint.log
