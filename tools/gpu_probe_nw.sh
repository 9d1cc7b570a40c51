# NW C4 timeline + per-phase cycle profile for a few variants (diagnostics; WF_TRACE adds clock reads)
WF_TRACE=1 timeout 300 python tools/perf_probe.py --fn seqcmp --dim 32768 --variants ${VARIANTS:-4,2,1 4,1,1 2,4,1 8,1,1 2,2,2} > gpurun_out/probe_nw.log 2>&1
python - <<'PY'
import json
for l in open("gpurun_out/probe_nw.log"):
    try: d = json.loads(l)
    except Exception: print(l.strip()); continue
    print(d.get("variant"), d.get("ms"), d.get("gcups"), "band_end", d.get("band_end_us", [])[:1], d.get("band_end_us", [])[-1:])
    print("  steady_entry", d.get("steady_entry_us_first_bands"))
    print("  ph0", d.get("nw_phase_cyc_per_row_band0"), "mid", d.get("nw_phase_cyc_per_row_mid"))
PY
