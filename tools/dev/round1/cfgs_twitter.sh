run twitter --workload twitter --steps 10 --warmup 3
