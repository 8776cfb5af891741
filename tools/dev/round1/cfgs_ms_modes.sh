run ms16_scan --sources 16 --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --mode scan
run lj_scan --steps 30 --warmup 5 --no-cpu-baseline --no-e2e --mode scan
run lj_scan_norl --steps 30 --warmup 5 --no-cpu-baseline --no-e2e --mode scan --relabel 0
run lj_opt --steps 30 --warmup 5 --no-cpu-baseline --no-e2e
