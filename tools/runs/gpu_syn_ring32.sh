timeout 1500 python -m pytest tests/test_parity_gpu.py tests/test_multiproc_gpu.py -m gpu -x -q -k "synthetic or staged" > gpurun_out/s2_tests.txt 2>&1; echo "rc=$?" >> gpurun_out/s2_tests.txt
timeout 900 python tools/ab_time.py --config C5a --rounds 4 ld256=- nowin=tools/abl_out/libwf_syn_nowin.so > gpurun_out/s2_c5a.txt 2>&1
timeout 900 python tools/ab_time.py --config C5b --rounds 3 ld256=- nowin=tools/abl_out/libwf_syn_nowin.so > gpurun_out/s2_c5b.txt 2>&1
timeout 900 python tools/ab_time.py --config C2 --rounds 3 ld256=- nowin=tools/abl_out/libwf_syn_nowin.so > gpurun_out/s2_c2.txt 2>&1
