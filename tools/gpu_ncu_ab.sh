# ncu --set full of one nw_kernel launch for experimental builds: NAMES="v5 ab3" bash tools/gpu_ncu_ab.sh
for n in ${NAMES}; do
  bash tools/ncu_probe_lib.sh tools/abl_out/libwf_$n.so gpurun_out/ncu_$n seqcmp ${DIM:-32768} ${VAR:-2,4,2} 2 > gpurun_out/ncu_$n.log 2>&1
  ncu -i gpurun_out/ncu_$n.ncu-rep --page raw --csv > gpurun_out/ncu_${n}_raw.csv 2>/dev/null
  ncu -i gpurun_out/ncu_$n.ncu-rep --page source --csv --print-source sass > gpurun_out/ncu_${n}_src.csv 2>/dev/null
  ls -la gpurun_out/ncu_$n*
done
