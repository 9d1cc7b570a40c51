# light-cell hand-off block UB (16 shipped vs 8), C5a / C5b, with the synthetic parity subset of the UB=8 build
WF_TEST_LIB=tools/abl_out/libwf_ub8.so timeout 900 python -m pytest tests/test_parity_gpu.py -m gpu -x -q -k "synthetic and not c5_full and not c5_prefix and not c2_full" > gpurun_out/ub_tests.txt 2>&1; echo "rc=$?" >> gpurun_out/ub_tests.txt
timeout 900 python tools/ab_time.py --config C5a --rounds 4 ub16=- ub8=tools/abl_out/libwf_ub8.so > gpurun_out/ub_c5a.txt 2>&1
timeout 900 python tools/ab_time.py --config C5b --rounds 3 ub16=- ub8=tools/abl_out/libwf_ub8.so > gpurun_out/ub_c5b.txt 2>&1
