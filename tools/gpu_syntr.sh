WF_TRACE=1 timeout 120 python tools/perf_probe.py --fn synthetic --tsize 10 --dsize 1 --dim 16384 --variants 1,1,1 1,4,1 2>&1 | python -c "
import json,sys
for l in sys.stdin:
    if l.startswith('{'):
        d=json.loads(l)
        if 'ms' not in d: print(d); continue
        s=d['band_start_us']; e=d['band_end_us']
        print(d['variant'], d['ms'], 'nbands', d['nbands'], 'starts', s[:4], s[-2:], 'ends', e[:3], e[-2:])
"
