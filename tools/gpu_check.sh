# One GPU call: parity tests, C4 bench, every config's bench line, ncu launch list of C4.
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
timeout 1500 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu.log 2>&1; echo "pytest rc=$?"
tail -3 gpurun_out/pytest_gpu.log
timeout 300 python bench.py > gpurun_out/bench_c4.json 2> gpurun_out/bench_c4.err; echo "bench rc=$?"
cat gpurun_out/bench_c4.json
rm -f gpurun_out/bench_all.jsonl
for c in C1 C2 C3 C5a C5b C5c C5d; do timeout 300 python bench.py --config $c --no-e2e-grid --steps 10 --warmup 3 >> gpurun_out/bench_all.jsonl 2>>gpurun_out/bench_all.err; done
cut -c1-300 gpurun_out/bench_all.jsonl
timeout 300 ncu --metrics gpu__time_duration.sum --clock-control none -c 60 --csv --log-file gpurun_out/c4_launches.csv python bench.py --steps 5 --warmup 3 --no-cpu-baseline --no-e2e-grid > gpurun_out/ncu_bench.log 2>&1; echo "ncu rc=$?"
timeout 300 python bench.py --impl reference --steps 3 --warmup 3 > gpurun_out/bench_ref.json 2>&1; echo "ref rc=$?"; cat gpurun_out/bench_ref.json | cut -c1-400
timeout 300 python -c "import __graft_entry__ as g; g.smoke(); print('smoke ok')" 2>&1 | tail -2
