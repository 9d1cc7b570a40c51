#!/usr/bin/env bash
# Build experimental libwf variants with parts of the NW steady loop disabled (WF_NW_ABL
# bitmask, see wf_nw.cuh) -- performance archaeology only; results are NOT correct grids.
set -e
cd "$(dirname "$0")/.."
mkdir -p /tmp/wfabl tools/abl_out
N=/usr/local/cuda/bin/nvcc
F="-gencode arch=compute_100a,code=sm_100a -O3 -lineinfo -std=c++17 -Xcompiler -fPIC --expt-relaxed-constexpr -Iinclude -Ipaper_conf_ppopp_mohantyc14_b200/csrc -DWF_MIN_VARIANTS"
$N $F -c paper_conf_ppopp_mohantyc14_b200/csrc/wf_api.cpp -o /tmp/wfabl/api.o
for A in "$@"; do
  ( $N $F -DWF_NW_ABL=$A -c paper_conf_ppopp_mohantyc14_b200/csrc/wf_sweep.cu -o /tmp/wfabl/sweep_$A.o &&
    $N -gencode arch=compute_100a,code=sm_100a -shared -cudart static -o tools/abl_out/libwf_abl_$A.so /tmp/wfabl/sweep_$A.o /tmp/wfabl/api.o ) &
done
wait
ls tools/abl_out
