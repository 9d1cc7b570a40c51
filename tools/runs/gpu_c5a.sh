# synthetic parity + C5a DRAM traffic (ncu dram bytes of one launch after warm-up) + C5a bench line
timeout 1500 python -m pytest tests/test_parity_gpu.py tests/test_multiproc_gpu.py -m gpu -x -q -k "synthetic" > gpurun_out/c5a_tests.txt 2>&1; echo "rc=$?" >> gpurun_out/c5a_tests.txt
timeout 600 python bench.py --config C5a --steps 10 --warmup 3 --no-cpu-baseline --no-e2e-grid > gpurun_out/c5a_bench.json 2> gpurun_out/c5a_bench.err
timeout 900 ncu --metrics dram__bytes_read.sum,dram__bytes_write.sum,gpu__time_duration.sum --clock-control none -k regex:syn_kernel -s 3 -c 1 --csv python tools/ncu_probe.py synthetic 16384 1,1,1 4 10 1 > gpurun_out/c5a_ncu.csv 2> gpurun_out/c5a_ncu.err
