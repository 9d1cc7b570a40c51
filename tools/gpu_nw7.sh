# NW v7: seqcmp parity, then C4 timing with the phase profile
timeout 600 python -m pytest tests -m gpu -x -q -k "seqcmp or watchdog" > gpurun_out/pytest_nw7.log 2>&1; echo "pytest rc=$?"
tail -3 gpurun_out/pytest_nw7.log | cut -c1-400
for lib in ""; do for f in 0 1; do
echo "== lib=$lib form=$f"
WF_LIB_OVERRIDE=$lib WF_NW7_FORM=$f timeout 120 python tools/perf_probe.py --fn seqcmp --dim 32768 --variants 4,2,1 8,1,1 2,4,1 > gpurun_out/probe_nw7.log 2>&1; cat gpurun_out/probe_nw7.log | cut -c1-300
WF_LIB_OVERRIDE=$lib WF_NW7_FORM=$f WF_TRACE=1 timeout 120 python tools/perf_probe.py --fn seqcmp --dim 32768 --variants 4,2,1 2>&1 | python -c "
import json,sys
for l in sys.stdin:
    if l.startswith('{'):
        d=json.loads(l); e=d['band_end_us']; print(d['ms'], 'band0_end', e[0], 'hop_us', round((e[-1]-e[0])/(8*(len(e)-1)),2), 'ph0', d['nw_phase_cyc_per_row_band0'], 'mid', d['nw_phase_cyc_per_row_mid'], 'raw', d['raw32_band0'][4:15])
    else: print(l[:200])
"
done; done
