# A/B of experimental libwf builds (tools/abl_out/libwf_NAME.so): parity subset + C4 timeline/phases
# usage: NAMES="base rot" VARIANTS="4,2,1" bash tools/gpu_ab.sh
for n in ${NAMES}; do
  echo "=== $n"
  if [ -n "${PARITY}" ]; then
    WF_LIB_OVERRIDE=tools/abl_out/libwf_$n.so timeout 120 python -m pytest tests/test_parity_gpu.py -m gpu -x -q -k "${PARITY}" 2>&1 | tail -2
  fi
  WF_LIB_OVERRIDE=tools/abl_out/libwf_$n.so WF_TRACE=${TRACE:-1} timeout 120 python tools/perf_probe.py --fn seqcmp --dim ${DIM:-32768} --variants ${VARIANTS:-4,2,1} > gpurun_out/ab_$n.log 2>&1
  python - "$n" <<'PY'
import json, sys
for l in open(f"gpurun_out/ab_{sys.argv[1]}.log"):
    try: d = json.loads(l)
    except Exception: print(l.strip()[:300]); continue
    print(d.get("variant"), d.get("ms"), d.get("gcups"), "band_end", d.get("band_end_us", [])[:1], d.get("band_end_us", [])[-1:])
    print("  steady_entry", d.get("steady_entry_us_first_bands", [])[:3], "io", d.get("io_fwd32_feed32_us"))
    print("  ph0", d.get("nw_phase_cyc_per_row_band0"), "mid", d.get("nw_phase_cyc_per_row_mid"))
    print("  slow", d.get("nw_slow_west_entries_polls_band0"), d.get("nw_slow_west_entries_polls_mid"))
PY
done
