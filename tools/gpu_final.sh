# round-end evidence pass (one gpurun call): GPU suite, smoke, bench lines, launch list, ncu of C4
set -x
timeout 2400 python -m pytest tests -m gpu -q > gpurun_out/fin_tests.txt 2>&1; echo "rc=$?" >> gpurun_out/fin_tests.txt
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/fin_smoke.txt 2>&1; echo "rc=$?" >> gpurun_out/fin_smoke.txt
timeout 900 python bench.py > gpurun_out/fin_bench_c4.json 2> gpurun_out/fin_bench_c4.err
rm -f gpurun_out/fin_bench_all.jsonl
for c in C1 C2 C3 C5a C5b C5c C5d; do timeout 900 python bench.py --config $c --steps 10 --warmup 3 >> gpurun_out/fin_bench_all.jsonl 2>> gpurun_out/fin_bench_all.err; done
timeout 900 python bench.py --impl reference --steps 3 --warmup 3 > gpurun_out/fin_bench_ref.json 2> gpurun_out/fin_bench_ref.err
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file gpurun_out/fin_c4_launches.csv python bench.py --steps 20 --warmup 3 --no-cpu-baseline --no-e2e-grid > gpurun_out/fin_ncu_launch.log 2>&1
timeout 900 ncu --set full --clock-control none -k regex:nw8_kernel -s 3 -c 1 -o gpurun_out/fin_c4 python tools/ncu_probe.py seqcmp 32768 2,4,1 4 > gpurun_out/fin_ncu_full.log 2>&1
ncu -i gpurun_out/fin_c4.ncu-rep --page raw --csv > gpurun_out/fin_c4_raw.csv 2>/dev/null
ncu -i gpurun_out/fin_c4.ncu-rep --page details --csv > gpurun_out/fin_c4_details.csv 2>/dev/null
rm -f gpurun_out/fin_c4.ncu-rep
