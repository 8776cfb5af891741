# persisting L2 window only when the hot set fits the set-aside: refresh of the affected configs
timeout 900 python -m pytest tests -m gpu -q --timeout 300 > gpurun_out/pytest_gpu.log 2>&1; echo pytest rc=$?; tail -2 gpurun_out/pytest_gpu.log
run lj --steps 100 --warmup 5 --no-cpu-baseline
run twitter --workload twitter --steps 10 --warmup 5 --no-cpu-baseline
run orkut_k1e6 --workload orkut --ins 250000 --dele 750000 --steps 5 --warmup 3 --no-cpu-baseline
run ms16 --sources 16 --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --mode shared
source tools/cfgs_ms_shards.sh
