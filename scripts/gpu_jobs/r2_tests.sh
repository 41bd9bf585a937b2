#!/bin/bash
# round 2: full GPU suite + a short bench line
cd "$GRAFT_REPO_ROOT"
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv > gpurun_out/r2_smi.txt 2>&1
timeout 1500 python -m pytest tests -m gpu -x -q --timeout 600 -p no:cacheprovider > gpurun_out/r2_gputest.log 2>&1
echo "pytest rc=$?" >> gpurun_out/r2_gputest.log
timeout 600 python bench.py --steps 5 --warmup 3 > gpurun_out/r2_bench.log 2>&1
echo "bench rc=$?" >> gpurun_out/r2_bench.log
tail -5 gpurun_out/r2_gputest.log
tail -c 1500 gpurun_out/r2_bench.log
