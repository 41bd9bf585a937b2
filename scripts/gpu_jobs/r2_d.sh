#!/bin/bash
# round 2 batch d: stencil fp32 pinning, PDL A/B, GPU suite, bench
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_tenants.py tests/test_gpu_bench_workload.py -k "stencil or c2" -x -q --timeout 300 -p no:cacheprovider > gpurun_out/r2d_stencil_tests.log 2>&1
echo "stencil tests rc=$?" >> gpurun_out/r2d_stencil_tests.log; tail -5 gpurun_out/r2d_stencil_tests.log
echo "== PDL on"; timeout 300 python scripts/stencil_iso.py stencil_tma stencil 2>&1 | tee gpurun_out/r2d_iso_pdl1.log
echo "== PDL off"; ACCEL_PDL=0 timeout 300 python scripts/stencil_iso.py stencil_tma stencil 2>&1 | tee gpurun_out/r2d_iso_pdl0.log
timeout 1500 python -m pytest tests -m gpu -x -q --timeout 600 -p no:cacheprovider > gpurun_out/r2d_gputest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r2d_gputest.log; tail -5 gpurun_out/r2d_gputest.log
timeout 300 python bench.py --steps 10 --warmup 3 > gpurun_out/r2d_bench.log 2>&1
tail -c 800 gpurun_out/r2d_bench.log
timeout 600 python scripts/isolated.py --reps 10 bfs cutcp stencil tpacf histo spmv sgemm mriq > gpurun_out/r2d_isolated.log 2>&1
