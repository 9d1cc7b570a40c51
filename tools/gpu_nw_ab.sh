# same-box A/B of NW builds: parity subset of the in-tree build, WF_TRACE timelines and interleaved timing
# usage: bash tools/gpu_nw_ab.sh NAME=lib ...   (lib '-' = in-tree)
timeout 1200 python -m pytest tests/test_parity_gpu.py tests/test_multiproc_gpu.py tests/test_abi_gpu.py -m gpu -x -q -k "seqcmp or smith or abi or multiproc or link or connect" > gpurun_out/ab_tests.txt 2>&1; echo "tests rc=$?" >> gpurun_out/ab_tests.txt
for nb in "$@"; do
  n=${nb%%=*}; l=${nb#*=}
  if [ "$l" = "-" ]; then WF_TRACE=1 timeout 300 python tools/nw8_probe.py trace 32768 > gpurun_out/ab_trace_$n.txt 2>&1
  else WF_TRACE=1 WF_PROBE_LIB=$l timeout 300 python tools/nw8_probe.py trace 32768 > gpurun_out/ab_trace_$n.txt 2>&1; fi
done
timeout 900 python tools/ab_time.py --rounds 4 "$@" > gpurun_out/ab.txt 2>&1
