run lj --steps 30 --warmup 5 --no-cpu-baseline --no-e2e
run orkut --workload orkut --steps 10 --warmup 3 --no-cpu-baseline --no-e2e
run twitter --workload twitter --steps 5 --warmup 3 --no-e2e
