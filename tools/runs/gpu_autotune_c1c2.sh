# autotune refresh for C1 and C2 on the final kernels
for c in C1 C2; do
  timeout 1500 python tools/autotune.py --config $c --reps 7 --out gpurun_out/autotune_$c.json > gpurun_out/autotune_$c.log 2>&1
  echo "$c rc=$?" >> gpurun_out/autotune_rc2.txt
done
