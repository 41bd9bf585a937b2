#!/bin/bash
# f2 at paper shape: seeded ordered tuples WITH repetition of the 8 tenants
# (PAPER.md lines 857-867), 1000 4-mixes and 500 8-mixes, NATIVE / RESOLVE / STATIC
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
timeout 2400 python scripts/mixes.py --config f2 --repeat --k 4 --n 1000 --reps 2 --seed 2024 --out gpurun_out/r2_f2_k4.json > gpurun_out/r2_f2_k4.log 2>&1
tail -1 gpurun_out/r2_f2_k4.log | cut -c 1-1500
timeout 2400 python scripts/mixes.py --config f2 --repeat --k 8 --n 500 --reps 2 --seed 2025 --out gpurun_out/r2_f2_k8.json > gpurun_out/r2_f2_k8.log 2>&1
tail -1 gpurun_out/r2_f2_k8.log | cut -c 1-1500
