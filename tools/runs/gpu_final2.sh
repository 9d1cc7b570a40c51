# final pass after the wf_syn changes: GPU suite, smoke, bench lines of every config
timeout 2400 python -m pytest tests -m gpu -q > gpurun_out/fin2_tests.txt 2>&1; echo "rc=$?" >> gpurun_out/fin2_tests.txt
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/fin2_smoke.txt 2>&1; echo "rc=$?" >> gpurun_out/fin2_smoke.txt
rm -f gpurun_out/fin2_bench_all.jsonl
for c in C1 C2 C3 C5a C5b C5c C5d; do timeout 900 python bench.py --config $c --steps 10 --warmup 3 >> gpurun_out/fin2_bench_all.jsonl 2>> gpurun_out/fin2_bench_all.err; done
timeout 900 python bench.py > gpurun_out/fin2_bench_c4.json 2> gpurun_out/fin2_bench_c4.err
