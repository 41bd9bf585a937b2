#!/bin/bash
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_tenants.py -k "bit_exact" -q -x --timeout 300 -p no:cacheprovider 2>&1 | tail -3
timeout 300 python scripts/stencil_iso.py stencil_bulk stencil 2>&1 | tee gpurun_out/r2s_iso.log
timeout 600 python scripts/diag_tma.py --reps 2 --sweeps 40 --kernel stencil_bulk --combos=-,bfs,bfs+cutcp+tpacf 2>&1 | tee gpurun_out/r2s_diag_bulk.log
timeout 300 python scripts/isolated.py --reps 6 gridding 2>&1 | cut -c 1-500
