# synthetic-kernel A/B (C5a and C2): parity of each build on small grids, interleaved timing
for nb in "$@"; do
  n=${nb%%=*}; l=${nb#*=}
  if [ "$l" != "-" ]; then export WF_TEST_LIB=$l; else unset WF_TEST_LIB; fi
  timeout 900 python -m pytest tests/test_parity_gpu.py -m gpu -x -q -k "synthetic and not c5_full and not c5_prefix and not c2_full" > gpurun_out/synab_tests_$n.txt 2>&1; echo "rc=$?" >> gpurun_out/synab_tests_$n.txt
done
unset WF_TEST_LIB
timeout 900 python tools/ab_time.py --config C5a --rounds 4 "$@" > gpurun_out/synab_c5a.txt 2>&1
timeout 900 python tools/ab_time.py --config C2 --rounds 3 "$@" > gpurun_out/synab_c2.txt 2>&1
timeout 900 python tools/ab_time.py --config C5c --rounds 2 "$@" > gpurun_out/synab_c5c.txt 2>&1
timeout 900 python tools/ab_time.py --config C5b --rounds 3 "$@" > gpurun_out/synab_c5b.txt 2>&1
