# ncu source-level stall sampling of one C4 launch of the in-tree NW kernel (tools/ncu_probe.py)
# -> gpurun_out/st9_g8_{raw,sass,cs}.csv for tools/ncu_region.py / tools/ncu_src_top.py
g=8
timeout 900 ncu --set full --clock-control none --import-source on -k regex:nw8_kernel -s 2 -c 1 -o gpurun_out/st9_g$g python tools/ncu_probe.py seqcmp 32768 2,4,1 3 0 0 0 0 > gpurun_out/st9_g$g.log 2>&1
echo "ncu rc=$?"
ncu -i gpurun_out/st9_g$g.ncu-rep --page raw --csv > gpurun_out/st9_g${g}_raw.csv 2>/dev/null
ncu -i gpurun_out/st9_g$g.ncu-rep --page source --csv --print-source sass > gpurun_out/st9_g${g}_sass.csv 2>/dev/null
ncu -i gpurun_out/st9_g$g.ncu-rep --page source --csv --print-source cuda,sass > gpurun_out/st9_g${g}_cs.csv 2>/dev/null
rm -f gpurun_out/st9_g$g.ncu-rep
