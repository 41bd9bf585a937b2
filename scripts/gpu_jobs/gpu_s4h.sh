# smoke() on the final build + ncu full of cutcp persistent (9 CTAs/SM) and native
python -m paper_conf_cgo_margiolaso16_b200.build > /dev/null 2>&1
timeout 300 python -c "import __graft_entry__ as g; g.smoke(); print('smoke ok')" 2>&1 | tail -2
timeout 300 ncu --set full --clock-control none --import-source on -k regex:accel_persistent -s 1 -c 1 -o gpurun_out/s4h_cutcp_static python scripts/profile_one.py cutcp persistent default > /dev/null 2>&1
timeout 300 ncu --set full --clock-control none --import-source on -k regex:accel_native -s 1 -c 1 -o gpurun_out/s4h_cutcp_native python scripts/profile_one.py cutcp native default > /dev/null 2>&1
ls gpurun_out
