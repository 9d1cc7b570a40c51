for c in C5d C5c C5b; do timeout 900 python tools/autotune.py --config $c --reps 3 --out gpurun_out/autotune_$c.json 2>&1 | grep best | cut -c1-250; done
