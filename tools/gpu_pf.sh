for lib in tools/abl_out/libwf_rx0.so tools/abl_out/libwf_pf0.so tools/abl_out/libwf_rot.so; do
echo "== $lib"
WF_LIB_OVERRIDE=$lib timeout 300 python -m pytest tests/test_parity_gpu.py -m gpu -x -q -k "seqcmp_dims or seqcmp_c4" 2>&1 | tail -1
WF_LIB_OVERRIDE=$lib timeout 300 python tools/perf_probe.py --fn seqcmp --dim 32768 --variants 4,2,1 4,1,1 2>&1 | cut -c1-150
done
