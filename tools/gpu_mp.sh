timeout 900 python -m pytest tests/test_multiproc_gpu.py -m gpu -x -q > gpurun_out/pytest_mp.log 2>&1; echo "pytest rc=$?"; tail -30 gpurun_out/pytest_mp.log | cut -c1-300
