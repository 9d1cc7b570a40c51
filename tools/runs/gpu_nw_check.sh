# parity subset + C4 trace + bench of the in-tree NW kernel (one gpurun call)
timeout 1200 python -m pytest tests/test_parity_gpu.py -m gpu -x -q -k "seqcmp or smith" > gpurun_out/vr_tests.txt 2>&1; echo "tests rc=$?" >> gpurun_out/vr_tests.txt
WF_TRACE=1 timeout 300 python tools/nw8_probe.py trace 32768 > gpurun_out/vr_trace.txt 2>&1
timeout 600 python bench.py --steps 50 --warmup 5 > gpurun_out/vr_bench.json 2> gpurun_out/vr_bench.err
