set -x
NCU=ncu
# launch list (serialised, cold-ish): stencil default 3 sweeps each mode
$NCU --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_stencil.csv python scripts/profile_one.py stencil native default sweeps=3 > /dev/null 2>&1
$NCU --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/launches_stencil_p.csv python scripts/profile_one.py stencil persistent default sweeps=3 > /dev/null 2>&1
# full set on one stencil launch, each mode
$NCU --set full --clock-control none --import-source on -k regex:accel_native -s 3 -c 1 -o gpurun_out/stencil_native python scripts/profile_one.py stencil native default sweeps=3 > gpurun_out/ncu_sn.log 2>&1
$NCU --set full --clock-control none --import-source on -k regex:accel_persistent -s 3 -c 1 -o gpurun_out/stencil_persist python scripts/profile_one.py stencil persistent default sweeps=3 > gpurun_out/ncu_sp.log 2>&1
$NCU --set full --clock-control none --import-source on -k regex:accel_native -s 3 -c 1 -o gpurun_out/histo_native python scripts/profile_one.py histo native default iters=3 > gpurun_out/ncu_hn.log 2>&1
ls -la gpurun_out
