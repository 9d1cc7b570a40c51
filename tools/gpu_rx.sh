for lib in tools/abl_out/libwf_rx0.so tools/abl_out/libwf_rx.so; do
WF_LIB_OVERRIDE=$lib timeout 600 python -m pytest tests/test_parity_gpu.py -m gpu -x -q -k "nash and not rectangular and not strategy and not band" 2>&1 | tail -1
WF_LIB_OVERRIDE=$lib timeout 300 python tools/perf_probe.py --fn nash --dim 4096 --variants 1,2,1 2>&1 | cut -c1-150
done
