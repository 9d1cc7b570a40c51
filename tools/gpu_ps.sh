# Plane-split synthetic kernel (kernel=8) vs the defaults' choice: parity tests, then interleaved timings
timeout 600 python -m pytest tests/test_parity_gpu.py -m gpu -x -q -k "plane_split or c5_prefix" > gpurun_out/ps_pytest.log 2>&1; echo "pytest rc=$?"; tail -3 gpurun_out/ps_pytest.log
for i in 1 2; do
  for cfg in "16384 1000 5 1,4,1,4 1,1,1,7 1,1,1,8" "16384 100 5 1,4,1,4 1,1,1,7 1,1,1,8" "16384 10 5 1,1,1,7 1,1,1,8" "16384 1000 2 1,1,1,7 1,1,1,8" "16384 1000 3 1,2,1,4 1,1,1,7 1,1,1,8" "16384 1000 4 1,2,1,4 1,1,1,7 1,1,1,8"; do
    set -- $cfg
    dim=$1; t=$2; d=$3; shift 3
    printf "dim=%s t=%s d=%s: " $dim $t $d
    timeout 300 python tools/perf_probe.py --fn synthetic --dim $dim --tsize $t --dsize $d --variants "$@" --reps 3 2>&1 | grep '^{' | python -c "import json,sys; [print(json.loads(l).get('variant'), json.loads(l).get('ms', json.loads(l).get('error'))) for l in sys.stdin]" | tr '\n' ' '
    echo
  done
done
