# ncu source-level stall sampling of one C5a launch (syn_kernel) -> gpurun_out/sts_C5a_{sass,cs}.csv
timeout 900 ncu --set full --clock-control none --import-source on -k regex:syn_kernel -s 3 -c 1 -o gpurun_out/sts_C5a python tools/ncu_probe.py synthetic 16384 1,1,1 4 10 1 > gpurun_out/sts_C5a.log 2>&1
echo "ncu rc=$?"
ncu -i gpurun_out/sts_C5a.ncu-rep --page source --csv --print-source sass > gpurun_out/sts_C5a_sass.csv 2>/dev/null
ncu -i gpurun_out/sts_C5a.ncu-rep --page source --csv --print-source cuda,sass > gpurun_out/sts_C5a_cs.csv 2>/dev/null
rm -f gpurun_out/sts_C5a.ncu-rep
