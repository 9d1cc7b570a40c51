timeout 900 python -m pytest tests -m gpu -x -q -k "nash" > gpurun_out/pytest_nash.log 2>&1; echo "pytest rc=$?"; tail -2 gpurun_out/pytest_nash.log | cut -c1-300
timeout 300 python tools/perf_probe.py --fn nash --dim 4096 --variants 1,1,1 1,2,1 1,4,1 1,8,1 2>&1 | cut -c1-150
