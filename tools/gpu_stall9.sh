# ncu source-level stall sampling of one C4 launch for NW generations 8 and 9 (tools/ncu_probe.py)
for g in 8 9; do
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:nw8_kernel -s 2 -c 1 -o gpurun_out/st9_g$g python tools/ncu_probe.py seqcmp 32768 2,4,1 3 0 0 0 $g > gpurun_out/st9_g$g.log 2>&1
  echo "g$g ncu rc=$?"
  ncu -i gpurun_out/st9_g$g.ncu-rep --page raw --csv > gpurun_out/st9_g${g}_raw.csv 2>/dev/null
  ncu -i gpurun_out/st9_g$g.ncu-rep --page source --csv --print-source sass > gpurun_out/st9_g${g}_sass.csv 2>/dev/null
  ncu -i gpurun_out/st9_g$g.ncu-rep --page source --csv --print-source cuda,sass > gpurun_out/st9_g${g}_cs.csv 2>/dev/null
  rm -f gpurun_out/st9_g$g.ncu-rep
done
ls -la gpurun_out/st9_*
