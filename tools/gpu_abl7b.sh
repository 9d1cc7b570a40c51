WF_LIB_OVERRIDE=tools/abl_out/libwf_abl0.so WF_TRACE=1 timeout 120 python tools/perf_probe.py --fn seqcmp --dim 32768 --variants 4,2,1 2>&1 | python -c "
import json,sys
for l in sys.stdin:
    if l.startswith('{'):
        d=json.loads(l); print(d['ms'], d['nw_phase_cyc_per_row_band0']); print('b0', d['raw32_band0']); print('mid', d['raw32_mid'])
    else: print(l[:200])
"
