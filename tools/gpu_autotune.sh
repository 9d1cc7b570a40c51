timeout 2700 python tools/autotune.py --all --reps 5 --budget-s 300 > gpurun_out/autotune.log 2>&1; echo "autotune rc=$?"
grep '"best"' gpurun_out/autotune.log | cut -c1-300
mkdir -p gpurun_out/at; cp profiles/autotune_*.json gpurun_out/at/ 2>/dev/null; ls gpurun_out/at
