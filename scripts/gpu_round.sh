set -x
timeout 900 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu.log 2>&1; echo pytest=$?
tail -3 gpurun_out/pytest_gpu.log
timeout 600 python bench.py > gpurun_out/bench.log 2>&1; echo bench=$?
tail -c 600 gpurun_out/bench.log
timeout 300 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file gpurun_out/r01b_launches_bench.csv python bench.py --steps 2 --warmup 3 --no-modes > /dev/null 2>&1; echo ncu1=$?
timeout 600 ncu --set full --clock-control none --import-source on -k regex:k_prof_ -c 2 -o gpurun_out/r01b_prof_c4 python scripts/prof_kernels.py priv --reps 1 > gpurun_out/ncu_prof.log 2>&1; echo ncu2=$?
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_tls_ -c 2 -o gpurun_out/r01b_tls python scripts/prof_kernels.py tls --reps 1 > gpurun_out/ncu_tls.log 2>&1; echo ncu3=$?
ls -la gpurun_out
