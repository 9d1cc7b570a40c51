# autotune refresh for the final kernels: C4 and C5a / C5c (parity-gated, device-timed), profiles/autotune_*.json
for c in C4 C5a C5c; do
  timeout 1500 python tools/autotune.py --config $c --reps 5 --out gpurun_out/autotune_$c.json > gpurun_out/autotune_$c.log 2>&1
  echo "$c rc=$?" >> gpurun_out/autotune_rc.txt
done
