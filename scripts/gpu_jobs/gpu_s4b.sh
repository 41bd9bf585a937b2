# stencil with per-VG hoisted addressing: parity + isolated timing + ncu full
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
python -m paper_conf_cgo_margiolaso16_b200.build > /dev/null 2>&1
timeout 600 python -m pytest tests -m gpu -q -x -k "stencil or config1 or mix" 2>&1 | tail -3
timeout 120 python scripts/isolated.py stencil --reps 5 2>&1 | cut -c1-700
timeout 300 ncu --set full --clock-control none --import-source on -k regex:accel_persistent -s 10 -c 1 -o gpurun_out/s4b_stencil_static python scripts/profile_one.py stencil persistent default sweeps=12 > /dev/null 2>&1
timeout 300 ncu --set full --clock-control none --import-source on -k regex:accel_persistent -s 10 -c 1 -o gpurun_out/s4b_stencil_resolve python scripts/profile_one.py stencil resolve default sweeps=12 > /dev/null 2>&1
ls gpurun_out
