#!/bin/bash
# histo: native vs persistent (same 274 CTAs) -- one launch each under ncu --set full
ACCEL_NO_OCC_CAP=1 python scripts/isolated.py histo --reps 3 > gpurun_out/hn_iso.log 2>&1
ACCEL_NO_OCC_CAP=1 timeout 600 ncu --set full --clock-control none --kernel-name-base demangled -k 'regex:accel_native<accel::HistoT<\(bool\)1>' -s 5 -c 1 -o gpurun_out/hn_native python scripts/isolated.py histo --reps 1 --policy static > gpurun_out/hn_ncu1.log 2>&1
ACCEL_NO_OCC_CAP=1 timeout 600 ncu --set full --clock-control none --kernel-name-base demangled -k 'regex:accel_persistent<accel::HistoT<\(bool\)1>, \(bool\)0>' -s 5 -c 1 -o gpurun_out/hn_pers python scripts/isolated.py histo --reps 1 --policy static > gpurun_out/hn_ncu2.log 2>&1
