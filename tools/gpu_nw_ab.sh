WF_TRACE=1 WF_PROBE_LIB=tools/abl_out/libwf_old.so timeout 300 python tools/nw8_probe.py trace 32768 > gpurun_out/ab1_trace_old.txt 2>&1
WF_TRACE=1 timeout 300 python tools/nw8_probe.py trace 32768 > gpurun_out/ab1_trace_new.txt 2>&1
WF_TRACE=1 WF_PROBE_LIB=tools/abl_out/libwf_dpre48.so timeout 300 python tools/nw8_probe.py trace 32768 > gpurun_out/ab1_trace_d48.txt 2>&1
WF_TRACE=1 WF_PROBE_LIB=tools/abl_out/libwf_dpre64.so timeout 300 python tools/nw8_probe.py trace 32768 > gpurun_out/ab1_trace_d64.txt 2>&1
timeout 900 python tools/ab_time.py --rounds 4 old=tools/abl_out/libwf_old.so new=- d48=tools/abl_out/libwf_dpre48.so d64=tools/abl_out/libwf_dpre64.so > gpurun_out/ab1.txt 2>&1
