#!/usr/bin/env bash
# The race / liveness build: every kernel with -DWF_JITTER=1 (random producer /
# consumer back-offs at each hand-off protocol, wf_sweep.cuh::wf_jitter; the non-.aligned block
# barrier of wf_nw8.cu so that compute-sanitizer synccheck applies), in-tree objects
# elsewhere untouched:  tools/xbuild_jitter.sh -> tools/abl_out/libwf_jitter.so
#   WF_TEST_LIB=tools/abl_out/libwf_jitter.so python -m pytest tests -m gpu -k "..."
set -e
cd "$(dirname "$0")/.."
mkdir -p /tmp/wfj tools/abl_out
N=/usr/local/cuda/bin/nvcc
F="-gencode arch=compute_100a,code=sm_100a -O3 -lineinfo -std=c++17 -Xcompiler -fPIC --expt-relaxed-constexpr -Iinclude -Ipaper_conf_ppopp_mohantyc14_b200/csrc -DWF_JITTER=1 -DWF_NW8_UNALIGNED_BAR"
OBJS=""
for s in paper_conf_ppopp_mohantyc14_b200/csrc/*.cu paper_conf_ppopp_mohantyc14_b200/csrc/*.cpp; do
  o=/tmp/wfj/$(basename $s).o
  $N $F -c $s -o $o &
  OBJS="$OBJS $o"
done
wait
$N -gencode arch=compute_100a,code=sm_100a -shared -cudart static -o tools/abl_out/libwf_jitter.so $OBJS
echo tools/abl_out/libwf_jitter.so
