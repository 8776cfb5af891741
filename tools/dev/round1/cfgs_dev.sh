run lj --steps 20 --warmup 3 --no-cpu-baseline
run orkut_k1e4 --workload orkut --steps 10 --warmup 3 --cpu-budget-s 20
run ms16 --sources 16 --steps 5 --warmup 3 --no-cpu-baseline --no-e2e
