# synthetic kernel (wf_syn.cu): parity, then per-config timings vs the generic sweep
timeout 900 python -m pytest tests -m gpu -x -q -k "synthetic" > gpurun_out/pytest_syn.log 2>&1; echo "pytest rc=$?"
tail -3 gpurun_out/pytest_syn.log | cut -c1-600
for c in C2 C5a C5b C5c C5d; do
  timeout 300 python bench.py --config $c --no-cpu-baseline --no-e2e-grid --steps 5 --warmup 3 2>/dev/null | python -c "import json,sys; d=json.loads(sys.stdin.read()); print('$c', d['value'], d['ms_per_step'], d['config'].get('warps'), d['config'].get('lane_cols'))"
done
for c in C2; do
  WF_SYN_IMPL=4 timeout 300 python bench.py --config $c --no-cpu-baseline --no-e2e-grid --steps 5 --warmup 3 2>/dev/null | python -c "import json,sys; d=json.loads(sys.stdin.read()); print('old $c', d['value'], d['ms_per_step'])"
done
timeout 120 python tools/perf_probe.py --fn synthetic --tsize 10 --dsize 1 --dim 16384 --variants 1,1,1 1,2,1 1,4,1 2,2,1 2>&1 | cut -c1-200
timeout 120 python tools/perf_probe.py --fn synthetic --tsize 10 --dsize 5 --dim 16384 --variants 1,1,1 1,2,1 2,2,1 2>&1 | cut -c1-200
