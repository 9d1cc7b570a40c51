# ncu --set full + source-level stall sampling of the dominant kernel (C4 NW generation 8, C5a synthetic),
# exported as raw / SASS / CUDA-source csv for tools/ncu_flag_stall.py (stall-on-flag fraction)
for c in C4 C5a; do
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:"nw8_kernel|nw_kernel|syn_kernel" -s 3 -c 1 -o gpurun_out/st_$c python bench.py --config $c --steps 1 --warmup 3 --no-cpu-baseline --no-e2e-grid > gpurun_out/st_$c.log 2>&1
  echo "$c ncu rc=$?"
  ncu -i gpurun_out/st_$c.ncu-rep --page raw --csv > gpurun_out/st_${c}_raw.csv 2>/dev/null
  ncu -i gpurun_out/st_$c.ncu-rep --page source --csv --print-source sass > gpurun_out/st_${c}_sass.csv 2>/dev/null
  ncu -i gpurun_out/st_$c.ncu-rep --page source --csv --print-source cuda,sass > gpurun_out/st_${c}_cs.csv 2>/dev/null
  ncu -i gpurun_out/st_$c.ncu-rep --page source --csv --print-source cuda > gpurun_out/st_${c}_cuda.csv 2>/dev/null
  rm -f gpurun_out/st_$c.ncu-rep
done
ls -la gpurun_out/st_*
