# ncu --set full of the dominant kernel of each config (one launch after warm-up), raw csv exported
for c in C4 C5a C3 C2 C1; do
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:"nw_kernel|syn_kernel|nash_kernel" -s 3 -c 1 -o gpurun_out/ncu_full_$c python bench.py --config $c --steps 1 --warmup 3 --no-cpu-baseline --no-e2e-grid > gpurun_out/ncu_full_$c.log 2>&1
  echo "$c ncu rc=$?"
  ncu -i gpurun_out/ncu_full_$c.ncu-rep --page raw --csv > gpurun_out/ncu_full_${c}_raw.csv 2>/dev/null; rm -f gpurun_out/ncu_full_$c.ncu-rep
done
ls -la gpurun_out/ncu_full_*raw.csv
