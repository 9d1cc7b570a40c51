# Interleaved A/B of the wf_syn feeder back-off (WF_SYN_FEED_NS 64 / 0 / 16) on C5a, C5b, C2, C5c
for i in 1 2; do
  for n in fb f0 f16; do
    for cfg in "16384 10 1" "16384 10 5" "2048 100 1" "16384 1000 1"; do
      set -- $cfg
      printf "%s dim=%s t=%s d=%s " "$n" $1 $2 $3
      WF_LIB_OVERRIDE=tools/abl_out/libwf_$n.so timeout 120 python tools/perf_probe.py --fn synthetic --dim $1 --tsize $2 --dsize $3 --variants 1,1,1 --reps 5 2>&1 | grep '^{' | python -c "import json,sys; [print(json.loads(l).get('ms')) for l in sys.stdin]" | tr '\n' ' '
      echo
    done
  done
done
