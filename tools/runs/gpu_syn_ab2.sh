# heavy-cell synthetic A/B (C5c, C5d) + the synthetic parity subset of the in-tree build
timeout 900 python -m pytest tests/test_parity_gpu.py -m gpu -x -q -k "synthetic and not c5_full and not c5_prefix and not c2_full" > gpurun_out/synab2_tests.txt 2>&1; echo "rc=$?" >> gpurun_out/synab2_tests.txt
timeout 1200 python -m pytest tests/test_parity_gpu.py -m gpu -x -q -k "c5_full or tsize1000" > gpurun_out/synab2_tests_full.txt 2>&1; echo "rc=$?" >> gpurun_out/synab2_tests_full.txt
timeout 900 python tools/ab_time.py --config C5c --rounds 2 "$@" > gpurun_out/synab2_c5c.txt 2>&1
timeout 1500 python tools/ab_time.py --config C5d --rounds 2 "$@" > gpurun_out/synab2_c5d.txt 2>&1
timeout 900 python tools/ab_time.py --config C5a --rounds 2 "$@" > gpurun_out/synab2_c5a.txt 2>&1
