# one GPU call: tests, bench, ncu launch list and captures (outputs under gpurun_out/)
set -x
timeout 900 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu.log 2>&1; echo pytest=$?
tail -3 gpurun_out/pytest_gpu.log
timeout 600 python bench.py > gpurun_out/bench.log 2>&1; echo bench=$?
timeout 300 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none -k regex:"k_" --csv --log-file gpurun_out/launches_bench.csv python bench.py --steps 5 --warmup 3 --no-modes > /dev/null 2>&1; echo ncu1=$?
timeout 600 ncu --set full --clock-control none --import-source on -k regex:"k_doall|k_priv" -c 3 -o gpurun_out/ncu_stream python scripts/prof_kernels.py all --reps 1 > gpurun_out/ncu_stream.log 2>&1; echo ncu2=$?
timeout 600 ncu --set full --clock-control none --import-source on -k regex:"k_prof_" -c 4 -o gpurun_out/ncu_prof python scripts/prof_kernels.py priv --reps 1 > gpurun_out/ncu_prof.log 2>&1; echo ncu3=$?
ls -la gpurun_out
