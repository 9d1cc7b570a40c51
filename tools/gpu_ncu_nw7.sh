# ncu --set full + source counters of one nw7_kernel launch (C4 shape), exported for reading here
N=${N:-nw7}
timeout 900 ncu --set full --clock-control none --import-source on -k regex:nw7_kernel -s 2 -c 1 -o gpurun_out/ncu_$N python tools/ncu_probe.py seqcmp ${DIM:-32768} ${VAR:-4,2,1} 3 > gpurun_out/ncu_$N.log 2>&1
echo "ncu rc=$?"; tail -3 gpurun_out/ncu_$N.log
ncu -i gpurun_out/ncu_$N.ncu-rep --page raw --csv > gpurun_out/ncu_${N}_raw.csv 2>/dev/null
ncu -i gpurun_out/ncu_$N.ncu-rep --page source --csv --print-source sass > gpurun_out/ncu_${N}_src.csv 2>/dev/null
ls -la gpurun_out/ncu_$N*
