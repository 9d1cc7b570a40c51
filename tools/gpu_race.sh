# Race and liveness evidence, one GPU:
#  1. compute-sanitizer memcheck / racecheck / synccheck over a small instance of every kernel family
#     (tools/sanitize_cases.py, each checked against the oracle), one log per tool, run on the
#     jitter build (tools/xbuild_jitter.sh -- it also carries the synccheck-clean barrier form);
#  2. the GPU parity tests against the jitter build (tools/xbuild_jitter.sh: random producer /
#     consumer back-offs at every hand-off protocol, wf_sweep.cuh::wf_jitter).
CASES=$(python tools/sanitize_cases.py --list)
for tool in memcheck racecheck synccheck; do
  : > gpurun_out/san_$tool.txt
  for c in $CASES; do
    echo "=== $tool $c" >> gpurun_out/san_$tool.txt
    WF_PROBE_LIB=tools/abl_out/libwf_jitter.so timeout 600 compute-sanitizer --tool $tool --print-limit 10 \
      python tools/sanitize_cases.py $c >> gpurun_out/san_$tool.txt 2>&1
    echo "rc=$?" >> gpurun_out/san_$tool.txt
  done
done
WF_TEST_LIB=tools/abl_out/libwf_jitter.so timeout 1500 python -m pytest tests -m gpu -q -k "not maximum_dim and not c4_full and not c5_full and not c3_prefix and not c5_prefix" > gpurun_out/jitter_tests.txt 2>&1
echo "jitter tests rc=$?" >> gpurun_out/jitter_tests.txt
