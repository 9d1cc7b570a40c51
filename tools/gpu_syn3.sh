timeout 900 python -m pytest tests -m gpu -x -q -k "synthetic or multiproc" > gpurun_out/pytest_syn.log 2>&1; echo "pytest rc=$?"; tail -3 gpurun_out/pytest_syn.log | cut -c1-300
for c in C2 C5a C5b C5c C5d; do
  timeout 300 python bench.py --config $c --no-cpu-baseline --no-e2e-grid --steps 5 --warmup 3 2>/dev/null | python -c "import json,sys; d=json.loads(sys.stdin.read()); print('$c', round(d['value'],3), round(d['ms_per_step'],3), d['config'].get('warps'), d['config'].get('lane_cols'))"
done
