# session 3q: C3, C4, f2 with the current build
export ACCEL_DEBUG_OFF=1
timeout 900 python scripts/mixes.py --config c3 --reps 3 --modes resolve,static --out gpurun_out/c3_pairs.json > gpurun_out/c3.log 2>&1; grep SUMMARY gpurun_out/c3.log | cut -c1-500
timeout 600 python scripts/mixes.py --config c4 --reps 5 --modes resolve,static --out gpurun_out/c4.json > gpurun_out/c4.log 2>&1; grep -E "^(native|resolve|static) " gpurun_out/c4.log | cut -c1-200
timeout 900 python scripts/mixes.py --config f2 --k 4 --n 40 --reps 3 --modes resolve,static --out gpurun_out/f2_k4.json > gpurun_out/f2.log 2>&1; grep SUMMARY gpurun_out/f2.log
