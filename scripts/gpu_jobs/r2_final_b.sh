#!/bin/bash
# Final round-2 evidence, part B: mixes with the profile-guided mode added
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
timeout 2400 python scripts/mixes.py --config f2 --repeat --k 4 --n 1000 --reps 2 --seed 2024 --out gpurun_out/fb_f2_k4.json > gpurun_out/fb_f2_k4.log 2>&1
timeout 1800 python scripts/mixes.py --config f2 --repeat --k 8 --n 500 --reps 2 --seed 2025 --out gpurun_out/fb_f2_k8.json > gpurun_out/fb_f2_k8.log 2>&1
timeout 900 python scripts/mixes.py --config c3 --reps 3 --out gpurun_out/fb_c3.json > gpurun_out/fb_c3.log 2>&1
timeout 600 python scripts/mixes.py --config c4 --reps 5 --out gpurun_out/fb_c4.json > gpurun_out/fb_c4.log 2>&1
