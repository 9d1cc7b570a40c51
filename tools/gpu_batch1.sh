set -x
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
timeout 900 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc=$?"
tail -3 gpurun_out/pytest_gpu.log
timeout 300 python bench.py > gpurun_out/bench_c4.json 2> gpurun_out/bench_c4.err; echo "bench rc=$?"
cat gpurun_out/bench_c4.json
for c in C1 C2 C3 C5a C5b C5c C5d; do timeout 300 python bench.py --config $c --no-cpu-baseline --no-e2e-grid --steps 10 --warmup 3 >> gpurun_out/bench_all.jsonl 2>>gpurun_out/bench_all.err; done
WF_TRACE=1 timeout 300 python tools/perf_probe.py --fn seqcmp --dim 32768 --variants 4,2,1 4,1,1 2,4,1 4,4,1 8,1,1 4,2,2 2,2,1 8,2,1 > gpurun_out/probe_nw.log 2>&1
cat gpurun_out/probe_nw.log | cut -c1-600
