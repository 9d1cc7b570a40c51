# size-aware NW default (cols <= 768: K=4 x 2 warps, 8-row strips): NW/SW parity subset, smoke, C1 bench, C1 autotune
timeout 1500 python -m pytest tests/test_parity_gpu.py tests/test_abi_gpu.py tests/test_multiproc_gpu.py -m gpu -x -q -k "seqcmp or smith or abi or multiproc" > gpurun_out/c1d_tests.txt 2>&1; echo "rc=$?" >> gpurun_out/c1d_tests.txt
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/c1d_smoke.txt 2>&1; echo "rc=$?" >> gpurun_out/c1d_smoke.txt
timeout 600 python bench.py --config C1 --steps 50 --warmup 5 > gpurun_out/c1d_bench.json 2> gpurun_out/c1d_bench.err
