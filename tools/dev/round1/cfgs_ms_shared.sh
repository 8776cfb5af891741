run ms16_shared --sources 16 --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --mode shared
run ms16_scan --sources 16 --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --mode scan
run ms256_shared --sources 256 --steps 3 --warmup 3 --no-cpu-baseline --no-e2e --mode shared
run lj_opt --steps 30 --warmup 5 --no-cpu-baseline --no-e2e
