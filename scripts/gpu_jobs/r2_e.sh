#!/bin/bash
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
timeout 600 python scripts/diag_tma.py --reps 2 2>&1 | tee gpurun_out/r2e_diag_tma.log
ACCEL_PDL=0 timeout 600 python scripts/diag_tma.py --reps 1 --sweeps 20 2>&1 | tee gpurun_out/r2e_diag_tma_pdl0.log
