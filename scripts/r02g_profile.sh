# round 2 (end): GPU tests, smoke, bench line, launch lists and full captures of the final code
set -x
mkdir -p gpurun_out
timeout 1800 python -m pytest tests -m gpu -x -q > gpurun_out/r02g_pytest_gpu.log 2>&1; echo pytest_rc=$?; tail -3 gpurun_out/r02g_pytest_gpu.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/r02g_smoke.log 2>&1; echo smoke_rc=$?
mkdir -p gpurun_out
timeout 1500 python bench.py > gpurun_out/r02g_bench.json 2> gpurun_out/r02g_bench.err
echo bench_rc=$?
M=gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum
ncu --metrics $M --clock-control none -k regex:"k_" -c 12 --csv --log-file gpurun_out/r02g_launches_bench_config2.csv python bench.py --steps 2 --warmup 3 --no-modes > /dev/null 2>&1
ncu --metrics $M --clock-control none -k regex:"k_" --csv --log-file gpurun_out/r02g_launches_sched3_d1.csv python scripts/sched3_once.py 0.01 > /dev/null 2>&1
ncu --metrics $M --clock-control none -k regex:"k_" --csv --log-file gpurun_out/r02g_launches_sched3_d0.csv python scripts/sched3_once.py 0.0 > /dev/null 2>&1
ncu --metrics $M --clock-control none -k regex:"k_" --csv --log-file gpurun_out/r02g_launches_waw_d1.csv python scripts/waw_once.py 0.01 > /dev/null 2>&1
ncu --metrics $M --clock-control none -k regex:"k_" --csv --log-file gpurun_out/r02g_launches_config5.csv python scripts/sched5_once.py > /dev/null 2>&1
ncu --metrics $M --clock-control none -k regex:"k_" --csv --log-file gpurun_out/r02g_launches_config4.csv python scripts/c4_call.py > /dev/null 2>&1
ncu --set full --clock-control none --import-source on -k regex:"k_bk_count|k_bk_scatter|k_bk_eval|k_tls_flow" -c 4 -o gpurun_out/r02g_sched3_full python scripts/sched3_once.py 0.01 > /dev/null 2>&1
ncu --set full --clock-control none --import-source on -k regex:"k_bk_pred|k_tls_flow_waw" -c 2 -o gpurun_out/r02g_waw_full python scripts/waw_once.py 0.01 > /dev/null 2>&1
ncu --set full --clock-control none --import-source on -k regex:"k_doall_gath|k_doall_scat" -c 2 -o gpurun_out/r02g_doall_full python scripts/sched3_once.py 0.0 > /dev/null 2>&1
ncu --set full --clock-control none -k regex:"k_doall_affine_tma" -c 1 -o gpurun_out/r02g_config2_full python bench.py --steps 2 --warmup 3 --no-modes > /dev/null 2>&1
ls -la gpurun_out
