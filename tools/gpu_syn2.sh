for v in st0 st1 st2; do
echo "== $v"
WF_LIB_OVERRIDE=tools/abl_out/libwf_$v.so WF_TRACE=1 timeout 120 python tools/perf_probe.py --fn synthetic --tsize 10 --dsize 1 --dim 16384 --variants 1,4,1 2>&1 | python -c "
import json,sys
for l in sys.stdin:
    if l.startswith('{'):
        d=json.loads(l)
        if 'ms' not in d: print(d); continue
        print(d['ms'], 'starts', d['band_start_us'][:4], 'ends', d['band_end_us'][:4])
    else: print(l[:300])
"
done
