run orkut_rl --workload orkut --steps 10 --warmup 3 --no-cpu-baseline --no-e2e
run orkut_norl --workload orkut --steps 10 --warmup 3 --no-cpu-baseline --no-e2e --no-relabel
run lj_norl --steps 30 --warmup 5 --no-cpu-baseline --no-e2e --no-relabel
run lj_rl --steps 30 --warmup 5 --no-cpu-baseline --no-e2e
