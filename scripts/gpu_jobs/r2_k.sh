#!/bin/bash
# f1 sharing-ratio rules on the paper-shape 4-mixes (first 300 of the f2 seed)
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
for al in 0 -0.25 -0.5 -1 0.5; do
  timeout 900 python scripts/mixes.py --config f2 --repeat --k 4 --n 300 --reps 2 --seed 2024 --modes resolve --alpha=$al --out gpurun_out/r2k_alpha_$al.json > gpurun_out/r2k_alpha_$al.log 2>&1
  echo "alpha $al"; tail -1 gpurun_out/r2k_alpha_$al.log | cut -c 1-700
done
