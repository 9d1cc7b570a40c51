# Nash launch bound (min resident CTAs per SM 8 shipped vs 12 / 16): parity of each build, C3 timing
for nb in base=- nash12=tools/abl_out/libwf_nash12.so nash16=tools/abl_out/libwf_nash16.so; do
  n=${nb%%=*}; l=${nb#*=}
  if [ "$l" != "-" ]; then export WF_TEST_LIB=$l; else unset WF_TEST_LIB; fi
  timeout 900 python -m pytest tests/test_parity_gpu.py -m gpu -x -q -k "nash" > gpurun_out/nmb_tests_$n.txt 2>&1; echo "rc=$?" >> gpurun_out/nmb_tests_$n.txt
done
unset WF_TEST_LIB
timeout 1200 python tools/ab_time.py --config C3 --rounds 3 base=- nash12=tools/abl_out/libwf_nash12.so nash16=tools/abl_out/libwf_nash16.so > gpurun_out/nmb_c3.txt 2>&1
