timeout 900 python -m pytest tests -m gpu -x -q -k "seqcmp or smith or watchdog or multiproc" > gpurun_out/pytest_sub.log 2>&1; echo "pytest rc=$?"; tail -3 gpurun_out/pytest_sub.log | cut -c1-300
timeout 120 python tools/perf_probe.py --fn seqcmp --dim 32768 --variants 4,2,1 4,1,1 8,1,1 2,4,1 2>&1 | cut -c1-200
WF_TRACE=1 timeout 120 python tools/perf_probe.py --fn seqcmp --dim 32768 --variants 4,2,1 2>&1 | python -c "
import json,sys
for l in sys.stdin:
    if l.startswith('{'):
        d=json.loads(l)
        e=d['band_end_us']; print(d['ms'], 'band0_end', e[0], 'hop_us', round((e[-1]-e[0])/(8*(len(e)-1)),2), 'ph0', d['nw_phase_cyc_per_row_band0'])
"
