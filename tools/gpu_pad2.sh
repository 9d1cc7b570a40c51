# Interleaved A/B of WF_SYN_PAD 0 / 2 on more synthetic shapes (one-warp variant 1,1,1)
for i in 1 2; do
  for n in pad0 pad2; do
    for cfg in "16384 1000 1" "16384 10 3" "16384 10 2" "16384 100 5" "4096 1000 5"; do
      set -- $cfg
      printf "%s dim=%s t=%s d=%s " "$n" $1 $2 $3
      WF_LIB_OVERRIDE=tools/abl_out/libwf_$n.so timeout 120 python tools/perf_probe.py --fn synthetic --dim $1 --tsize $2 --dsize $3 --variants 1,1,1 --reps 5 2>&1 | grep '^{' | python -c "import json,sys; [print(json.loads(l).get('ms')) for l in sys.stdin]" | tr '\n' ' '
      echo
    done
  done
done
