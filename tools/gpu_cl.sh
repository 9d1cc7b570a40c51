timeout 900 python -m pytest tests -m gpu -x -q -k "seqcmp_dims or smith or c4" > gpurun_out/pytest_cl.log 2>&1; echo "pytest rc=$?"; tail -2 gpurun_out/pytest_cl.log | cut -c1-300
WF_NW_CLUSTER=4 timeout 600 python -m pytest tests -m gpu -x -q -k "seqcmp_dims or c4 or local_slabs" > gpurun_out/pytest_cl4.log 2>&1; echo "pytest cl4 rc=$?"; tail -2 gpurun_out/pytest_cl4.log | cut -c1-300
for cl in 0 2 4; do
echo "== cluster=$cl"
WF_NW_CLUSTER=$cl WF_NW_CLUSTER_DEBUG=1 timeout 120 python tools/perf_probe.py --fn seqcmp --dim 32768 --variants 4,2,1 2>&1 | sort | uniq | cut -c1-200
done
