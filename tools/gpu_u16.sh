timeout 600 python -m pytest tests -m gpu -x -q -k "seqcmp or watchdog" > gpurun_out/pytest_nw.log 2>&1; echo "pytest rc=$?"; tail -2 gpurun_out/pytest_nw.log
WF_TRACE=1 timeout 120 python tools/perf_probe.py --fn seqcmp --dim 32768 --variants 4,2,1 2>&1 | python -c "
import json,sys
for l in sys.stdin:
    if l.startswith('{'):
        d=json.loads(l)
        e=d['band_end_us']; print(d['ms'], 'band0_end', e[0], 'hop_us', round((e[-1]-e[0])/(8*(len(e)-1)),2))
        print('steady_entry', d['steady_entry_us_first_bands']); print('fwd32/feed32', d['io_fwd32_feed32_us'])
"
timeout 120 python tools/perf_probe.py --fn seqcmp --dim 32768 --variants 4,2,1 4,1,1 8,1,1 2>&1 | cut -c1-200
