set -x
python bench.py > gpurun_out/bench_r02b.json 2> gpurun_out/bench_r02b.err; echo bench_rc=$?
tail -c 3000 gpurun_out/bench_r02b.json
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file gpurun_out/launches_r02b.csv python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu-baseline --extra-n 0 > gpurun_out/bench_ncu_r02b.log 2>&1; echo ncu_list_rc=$?
timeout 900 ncu --set full --clock-control none --import-source on -k regex:^k_sched$ -c 1 -o gpurun_out/sched46080_r02b python tools/profile_run.py 46080 sched > gpurun_out/ncu46080.log 2>&1; echo ncu46_rc=$?
timeout 600 ncu --set full --clock-control none --import-source on -k regex:^k_sched$ -c 1 -o gpurun_out/sched19200_r02b python tools/profile_run.py 19200 sched > gpurun_out/ncu19200.log 2>&1; echo ncu19_rc=$?
ls -la gpurun_out
