#!/usr/bin/env bash
# Experimental libwf build (reduced variant set, extra -D flags) for perf archaeology:
#   tools/xbuild.sh NAME -DFLAG=1 ...   ->  tools/abl_out/libwf_NAME.so  (use via WF_LIB_OVERRIDE)
set -e
cd "$(dirname "$0")/.."
NAME=$1; shift
mkdir -p /tmp/wfx tools/abl_out
N=/usr/local/cuda/bin/nvcc
F="-gencode arch=compute_100a,code=sm_100a -O3 -lineinfo -std=c++17 -Xcompiler -fPIC --expt-relaxed-constexpr -Iinclude -Ipaper_conf_ppopp_mohantyc14_b200/csrc -DWF_MIN_VARIANTS"
OBJS=""
for s in paper_conf_ppopp_mohantyc14_b200/csrc/*.cu paper_conf_ppopp_mohantyc14_b200/csrc/*.cpp; do
  o=/tmp/wfx/$(basename $s)_$NAME.o
  $N $F "$@" -c $s -o $o &
  OBJS="$OBJS $o"
done
wait
$N -gencode arch=compute_100a,code=sm_100a -shared -cudart static -o tools/abl_out/libwf_$NAME.so $OBJS
echo tools/abl_out/libwf_$NAME.so
