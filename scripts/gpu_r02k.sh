mkdir -p gpurun_out
timeout 1500 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu.log 2>&1; echo pytest=$?; tail -3 gpurun_out/pytest_gpu.log
timeout 300 python scripts/sched3_time.py > gpurun_out/sched3.log 2>&1; echo t=$?; cat gpurun_out/sched3.log
timeout 300 python scripts/waw_time.py > gpurun_out/waw_time.log 2>&1; echo waw=$?; cat gpurun_out/waw_time.log | tail -8
timeout 300 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none -k regex:"k_" --csv --log-file gpurun_out/launches_sched3_d1.csv python scripts/sched3_once.py 0.01 > /dev/null 2>&1; echo ncu=$?
