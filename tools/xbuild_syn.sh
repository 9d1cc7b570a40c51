#!/usr/bin/env bash
# Experimental libwf with only wf_syn.cu rebuilt under extra -D flags (perf A/B of the
# generation-8 NW kernel), linked with the in-tree objects of everything else:
#   tools/xbuild_syn.sh NAME -DWF_NW8_U=16 ...  ->  tools/abl_out/libwf_NAME.so  (WF_PROBE_LIB=... for tools/nw8_probe.py)
set -e
cd "$(dirname "$0")/.."
NAME=$1; shift
mkdir -p /tmp/wfx tools/abl_out
N=/usr/local/cuda/bin/nvcc
F="-gencode arch=compute_100a,code=sm_100a -O3 -lineinfo -std=c++17 -Xcompiler -fPIC --expt-relaxed-constexpr -Iinclude -Ipaper_conf_ppopp_mohantyc14_b200/csrc"
B=paper_conf_ppopp_mohantyc14_b200/_build
$N $F "$@" -c paper_conf_ppopp_mohantyc14_b200/csrc/wf_syn.cu -o /tmp/wfx/wf_syn_$NAME.o
OBJS=$(ls $B/*.o | grep -v wf_syn.cu.o)
$N -gencode arch=compute_100a,code=sm_100a -shared -cudart static -o tools/abl_out/libwf_$NAME.so $OBJS /tmp/wfx/wf_syn_$NAME.o
echo tools/abl_out/libwf_$NAME.so
