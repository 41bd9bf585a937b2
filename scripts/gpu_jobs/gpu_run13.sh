timeout 900 python -m pytest tests -m gpu -q -x -k "stencil or resolve or mix" 2>&1 | tail -3
timeout 600 python scripts/isolated.py stencil --reps 3 2>&1 | tail -2
NCU="ncu --set full --clock-control none --import-source on"
timeout 600 $NCU -k regex:accel_native -s 4 -c 1 -o gpurun_out/stencil_n6 python scripts/profile_one.py stencil native default sweeps=8 > /dev/null 2>&1
timeout 600 $NCU -k regex:accel_persistent -s 4 -c 1 -o gpurun_out/stencil_p6 python scripts/profile_one.py stencil persistent default sweeps=8 > /dev/null 2>&1
