# end-of-round refresh of every BASELINE config (CFGFILE for tools/bench_configs.sh)
run lj --steps 100 --warmup 5
run tiny --workload tiny --steps 20 --warmup 5
run orkut_k1e4 --workload orkut --steps 20 --warmup 5 --no-cpu-baseline
run orkut_k1e2 --workload orkut --ins 25 --dele 75 --steps 50 --warmup 5 --no-cpu-baseline
run orkut_k1e6 --workload orkut --ins 250000 --dele 750000 --steps 5 --warmup 3 --no-cpu-baseline
run twitter --workload twitter --steps 10 --warmup 5 --no-cpu-baseline
run ms256 --sources 256 --steps 10 --warmup 3 --no-cpu-baseline --no-e2e
run ms256_s0of8 --sources 256 --shard 0/8 --steps 10 --warmup 3 --no-cpu-baseline --no-e2e
run ms256_s0of4 --sources 256 --shard 0/4 --steps 10 --warmup 3 --no-cpu-baseline --no-e2e
run ms256_s0of2 --sources 256 --shard 0/2 --steps 10 --warmup 3 --no-cpu-baseline --no-e2e
