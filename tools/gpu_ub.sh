for lib in ""; do
echo "== $lib"
for spec in "10 1 16384" "10 5 16384" "100 1 2048" "1000 1 16384"; do set -- $spec
WF_LIB_OVERRIDE=$lib timeout 200 python tools/perf_probe.py --fn synthetic --tsize $1 --dsize $2 --dim $3 --variants 1,1,1 --reps 3 2>&1 | cut -c1-120
done; done
