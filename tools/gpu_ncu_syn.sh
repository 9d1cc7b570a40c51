N=syn
timeout 900 ncu --set full --clock-control none --import-source on -k regex:syn_kernel -s 1 -c 1 -o gpurun_out/ncu_$N python tools/ncu_probe.py synthetic 4096 1,4,1 2 10 1 > gpurun_out/ncu_$N.log 2>&1
echo "ncu rc=$?"; tail -3 gpurun_out/ncu_$N.log
ncu -i gpurun_out/ncu_$N.ncu-rep --page source --csv --print-source sass > gpurun_out/ncu_${N}_src.csv 2>/dev/null
ncu -i gpurun_out/ncu_$N.ncu-rep --page raw --csv > gpurun_out/ncu_${N}_raw.csv 2>/dev/null
