# v7 ablations (wrong grids, timing only) + FORM comparison, with the WF_TRACE phase profile
for f in 0 1; do for n in abl0 abl1 abl2 abl4 abl7; do
  echo "== $n form $f"
  WF_NW7_FORM=$f WF_LIB_OVERRIDE=tools/abl_out/libwf_$n.so WF_TRACE=1 timeout 120 python tools/perf_probe.py --fn seqcmp --dim 32768 --variants 4,2,1 2>&1 | python -c "
import json,sys
for l in sys.stdin:
    if l.startswith('{'):
        d=json.loads(l); e=d['band_end_us']; print(d['ms'], 'band0_end', e[0], 'hop_us', round((e[-1]-e[0])/(8*(len(e)-1)),2), 'ph0', d['nw_phase_cyc_per_row_band0'], 'mid', d['nw_phase_cyc_per_row_mid'])
    else: print(l[:200])
"
done; done
