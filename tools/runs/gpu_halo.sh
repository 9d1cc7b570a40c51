timeout 900 python -m pytest tests/test_parity_gpu.py -m gpu -x -q -k "halo or local_slabs or strips_local" > gpurun_out/halo_tests.txt 2>&1; echo "rc=$?" >> gpurun_out/halo_tests.txt
CUDA_DEVICE_MAX_CONNECTIONS=32 timeout 900 python tools/halo_ab.py 3 > gpurun_out/halo_ab.txt 2>&1
