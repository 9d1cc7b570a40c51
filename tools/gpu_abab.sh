# Interleaved A/B/A/B timing of experimental libwf builds (tools/abl_out/libwf_NAME.so) on C4,
# several rounds in one process each, so box-to-box clock differences cancel.
# usage: NAMES="old new" ROUNDS=4 bash tools/gpu_abab.sh
for i in $(seq 1 ${ROUNDS:-4}); do
  for n in ${NAMES}; do
    printf "%s " "$n"
    WF_LIB_OVERRIDE=tools/abl_out/libwf_$n.so timeout 120 python tools/perf_probe.py --fn seqcmp --dim ${DIM:-32768} --variants ${VARIANTS:-4,2,1} --reps ${REPS:-30} 2>&1 | tr '\n' ' '
    echo
  done
done
