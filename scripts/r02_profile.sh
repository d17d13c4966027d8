set -x
mkdir -p gpurun_out
timeout 1500 python bench.py > gpurun_out/bench_r02e.json 2> gpurun_out/bench_r02e.err
echo bench_rc=$?
# launch list of the bench command's first steps (cold, serialised) -- config 2 headline
ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none -k regex:"k_" -c 12 --csv --log-file gpurun_out/r02_launches_bench_config2.csv python bench.py --steps 2 --warmup 3 --no-modes > /dev/null 2>&1
# whole jp_schedule launch lists: config 3 (d = 1%, 10%), config 4, config 5
ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none -k regex:"k_" --csv --log-file gpurun_out/r02_launches_sched3_d1.csv python scripts/sched3_once.py 0.01 > /dev/null 2>&1
ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none -k regex:"k_" --csv --log-file gpurun_out/r02_launches_sched3_d10.csv python scripts/sched3_once.py 0.1 > /dev/null 2>&1
ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none -k regex:"k_" --csv --log-file gpurun_out/r02_launches_config4.csv python scripts/c4_call.py > /dev/null 2>&1
# full captures of the new kernels
ncu --set full --clock-control none --import-source on -k regex:"k_tls_flow|k_bk_scatter|k_bk_eval|k_bk_count" -c 4 -o gpurun_out/r02_sched3_full python scripts/sched3_once.py 0.01 > /dev/null 2>&1
ncu --set full --clock-control none --import-source on -k regex:"k_priv_tmp_2ph" -c 1 -o gpurun_out/r02_config4_full python scripts/c4_call.py > /dev/null 2>&1
ncu --set full --clock-control none -k regex:"k_doall_affine_tma" -c 1 -o gpurun_out/r02_config2_full python bench.py --steps 2 --warmup 3 --no-modes > /dev/null 2>&1
ls -la gpurun_out
