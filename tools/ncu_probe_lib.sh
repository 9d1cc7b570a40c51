#!/usr/bin/env bash
# ncu source-level capture of one nw_kernel launch using an experimental library build
LIB=$1; OUT=$2; shift 2
WF_LIB_OVERRIDE=$LIB timeout 600 ncu --set full --clock-control none --import-source on -k regex:nw_kernel -s 1 -c 1 -o $OUT python tools/ncu_probe.py "$@"
