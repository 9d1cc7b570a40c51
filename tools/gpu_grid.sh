timeout 2400 python tools/autotune.py --grid --reps 3 --out gpurun_out/tuner_sweep.json > gpurun_out/grid.log 2>&1; echo "grid rc=$?"; tail -2 gpurun_out/grid.log; grep -c '"ms"' gpurun_out/grid.log
