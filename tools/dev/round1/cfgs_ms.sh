run ms16 --sources 16 --steps 5 --warmup 3 --no-cpu-baseline --no-e2e
