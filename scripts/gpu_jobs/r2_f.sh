#!/bin/bash
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
for p in 0 1 2 3; do echo "== ACCEL_TMA_PROMO=$p"; ACCEL_TMA_PROMO=$p timeout 600 python scripts/diag_tma.py --reps 2 --sweeps 40 2>&1 | grep -v "co=cutcp\|co=tpacf"; done 2>&1 | tee gpurun_out/r2f_diag_promo.log
