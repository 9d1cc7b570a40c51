WF_LIB_OVERRIDE=tools/abl_out/libwf_tr.so WF_TRACE=1 timeout 120 python tools/perf_probe.py --fn seqcmp --dim 32768 --variants 4,2,1 2>&1 | python -c "
import json,sys
for l in sys.stdin:
    if l.startswith('{'):
        d=json.loads(l)
        if 'ms' not in d: print(d); continue
        b0=d['raw32_band0']; m=d['raw32_mid']
        print(d['ms'])
        print('steady_entry', d['steady_entry_us_first_bands'][:3]); print('fwd32/feed32', d['io_fwd32_feed32_us'][:3])
        print('raw band0 32..47', b0[:16])
"
