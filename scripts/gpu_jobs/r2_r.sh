#!/bin/bash
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_tenants2.py tests/test_gpu_tenants.py -k "gridding or pipeline" -q -x --timeout 300 -p no:cacheprovider 2>&1 | tail -15
timeout 300 python scripts/isolated.py --reps 6 gridding histo_pipeline 2>&1 | cut -c 1-700
