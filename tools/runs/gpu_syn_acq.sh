# wait_ctr acquire load vs volatile load + __threadfence_block (and UB 8 with the acquire form): parity + C5a / C5b / C2 timing
timeout 900 python -m pytest tests/test_parity_gpu.py -m gpu -x -q -k "synthetic and not c5_full and not c5_prefix and not c2_full" > gpurun_out/acq_tests.txt 2>&1; echo "rc=$?" >> gpurun_out/acq_tests.txt
timeout 900 python tools/ab_time.py --config C5a --rounds 4 acq=- fence=tools/abl_out/libwf_fence.so acq_ub8=tools/abl_out/libwf_acq_ub8.so > gpurun_out/acq_c5a.txt 2>&1
timeout 900 python tools/ab_time.py --config C5b --rounds 3 acq=- fence=tools/abl_out/libwf_fence.so > gpurun_out/acq_c5b.txt 2>&1
timeout 900 python tools/ab_time.py --config C2 --rounds 3 acq=- fence=tools/abl_out/libwf_fence.so > gpurun_out/acq_c2.txt 2>&1
