for f in 0 1; do
WF_NW_IMPL=7 WF_NW7_FORM=$f timeout 200 python tools/perf_probe.py --fn seqcmp --dim 32768 --variants 4,2,1 4,4,1 2,8,1 1,8,1 2,4,1 2>&1 | cut -c1-200
done
timeout 200 python tools/perf_probe.py --fn seqcmp --dim 32768 --variants 4,2,1 2>&1 | cut -c1-200
