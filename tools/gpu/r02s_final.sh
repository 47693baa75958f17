# final validation of the round-2 build: bench line, reference arm, GPU tests, sweep with
# bounds, ncu launch list + ncu --set full of k_sched at the bench sizes
export PYTHONUNBUFFERED=1
set -x
python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke_final.log 2>&1; echo smoke_rc=$?
python bench.py > gpurun_out/bench_final.json 2> gpurun_out/bench_final.err; echo bench_rc=$?
python bench.py --impl reference > gpurun_out/bench_ref_final.json 2>> gpurun_out/bench_final.err; echo ref_rc=$?
timeout 1200 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu_final.log 2>&1; echo pytest_rc=$?
timeout 900 python tools/sweep.py 4,6,8,10,12,16,20,24,32,48 > gpurun_out/sweep_final.jsonl 2> gpurun_out/sweep_final.err; echo sweep_rc=$?
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file gpurun_out/launches_final.csv python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu-baseline --extra-n 0 > gpurun_out/bench_ncu_final.log 2>&1; echo ncu_list_rc=$?
timeout 900 ncu --set full --clock-control none --import-source on -k 'regex:^k_sched$' -c 1 -o gpurun_out/sched46080_final python tools/profile_run.py 46080 sched > gpurun_out/ncu46080_final.log 2>&1; echo ncu46_rc=$?
timeout 600 ncu --set full --clock-control none --import-source on -k 'regex:^k_sched$' -c 1 -o gpurun_out/sched19200_final python tools/profile_run.py 19200 sched > gpurun_out/ncu19200_final.log 2>&1; echo ncu19_rc=$?
