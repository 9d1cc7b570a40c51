timeout 1500 python -m pytest tests/test_parity_gpu.py tests/test_multiproc_gpu.py -m gpu -x -q -k "synthetic or staged" > gpurun_out/s32_tests.txt 2>&1; echo "rc=$?" >> gpurun_out/s32_tests.txt
timeout 900 ncu --metrics dram__bytes_read.sum,dram__bytes_write.sum,gpu__time_duration.sum --clock-control none -k regex:syn_kernel -s 3 -c 1 --csv python tools/ncu_probe.py synthetic 16384 1,1,1 4 10 1 > gpurun_out/s32_ncu_c5a.csv 2> gpurun_out/s32_ncu.err
timeout 900 ncu --metrics dram__bytes_read.sum,dram__bytes_write.sum,gpu__time_duration.sum --clock-control none -k regex:syn_kernel -s 3 -c 1 --csv python tools/ncu_probe.py synthetic 16384 1,1,1 4 10 5 > gpurun_out/s32_ncu_c5b.csv 2>> gpurun_out/s32_ncu.err
timeout 900 python tools/ab_time.py --config C5a --rounds 4 new=- head=tools/abl_out/libwf_synhead.so > gpurun_out/s32_c5a.txt 2>&1
timeout 900 python tools/ab_time.py --config C5b --rounds 3 new=- head=tools/abl_out/libwf_synhead.so > gpurun_out/s32_c5b.txt 2>&1
timeout 900 python tools/ab_time.py --config C2 --rounds 3 new=- head=tools/abl_out/libwf_synhead.so > gpurun_out/s32_c2.txt 2>&1
