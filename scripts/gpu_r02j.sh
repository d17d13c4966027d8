mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_tls_fwd.py tests/test_gpu_flow_waw.py tests/test_gpu_fullsize.py -x -q > gpurun_out/pytest_j.log 2>&1; echo pytest=$?; tail -3 gpurun_out/pytest_j.log
timeout 300 python scripts/sched3_time.py > gpurun_out/sched3_ph.log 2>&1; echo t=$?; cat gpurun_out/sched3_ph.log
JP_FLOW_PHASED=0 timeout 300 python scripts/sched3_time.py > gpurun_out/sched3_noph.log 2>&1; echo t=$?; cat gpurun_out/sched3_noph.log
timeout 300 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none -k regex:"k_tls_flow" --csv --log-file gpurun_out/launches_flow_ph.csv python scripts/sched3_once.py 0.01 > /dev/null 2>&1; echo ncu=$?
