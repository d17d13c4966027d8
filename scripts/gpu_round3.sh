# one GPU call: full gpu tests, bench, launch list, ncu captures of the round-1d kernels
timeout 1500 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu.log 2>&1; echo pytest=$?; tail -3 gpurun_out/pytest_gpu.log
timeout 600 python bench.py > gpurun_out/bench.log 2>&1; echo bench=$?
timeout 300 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none -k regex:"k_" --csv --log-file gpurun_out/launches_bench.csv python bench.py --steps 5 --warmup 3 --no-modes > /dev/null 2>&1; echo ncu1=$?
timeout 600 ncu --set full --clock-control none --import-source on -k regex:"k_doall_spill" -c 1 -o gpurun_out/ncu_spill python scripts/prof_kernels.py spill --reps 2 > gpurun_out/ncu_spill.log 2>&1; echo ncu2=$?
timeout 600 ncu --set full --clock-control none --import-source on -k regex:"k_x_" -c 4 -o gpurun_out/ncu_exchange python scripts/prof_kernels.py exchange --reps 1 > gpurun_out/ncu_exchange.log 2>&1; echo ncu3=$?
ls gpurun_out
