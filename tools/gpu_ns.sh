for lib in "" tools/abl_out/libwf_ns64.so tools/abl_out/libwf_ns256.so tools/abl_out/libwf_ns1000.so; do
echo "== $lib"
WF_LIB_OVERRIDE=$lib timeout 200 python tools/perf_probe.py --fn nash --dim 4096 --variants 1,8,1 2>&1 | cut -c1-200
done
