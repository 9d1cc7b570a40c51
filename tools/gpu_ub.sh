# Interleaved A/B of the wf_syn hand-off block UB (light: C5a / C5b; medium: C2, dsize 5 tsize 100)
for i in 1 2; do
  for n in ub_base ub_l32 ub_l8; do
    for cfg in "16384 10 1" "16384 10 5"; do
      set -- $cfg
      printf "%s dim=%s t=%s d=%s " "$n" $1 $2 $3
      WF_LIB_OVERRIDE=tools/abl_out/libwf_$n.so timeout 120 python tools/perf_probe.py --fn synthetic --dim $1 --tsize $2 --dsize $3 --variants 1,1,1 --reps 5 2>&1 | grep '^{' | python -c "import json,sys; [print(json.loads(l).get('ms')) for l in sys.stdin]" | tr '\n' ' '
      echo
    done
  done
  for n in ub_base ub_m16 ub_m4; do
    for cfg in "2048 100 1" "16384 100 1"; do
      set -- $cfg
      printf "%s dim=%s t=%s d=%s " "$n" $1 $2 $3
      WF_LIB_OVERRIDE=tools/abl_out/libwf_$n.so timeout 120 python tools/perf_probe.py --fn synthetic --dim $1 --tsize $2 --dsize $3 --variants 1,1,1 --reps 5 2>&1 | grep '^{' | python -c "import json,sys; [print(json.loads(l).get('ms')) for l in sys.stdin]" | tr '\n' ' '
      echo
    done
  done
done
