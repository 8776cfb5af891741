mkdir -p gpurun_out
python -m paper_journals_pvldb_guolst17_b200.build || exit 1
[ -n "$NOTEST" ] || timeout 900 python -m pytest tests -m gpu -q -x --timeout 600 -k "shared or multi_source" > gpurun_out/pytest_ms.log 2>&1; echo pytest rc=$?; tail -3 gpurun_out/pytest_ms.log
CFGFILE=${CFGFILE:-tools/cfgs_ms_curve.sh} bash tools/bench_configs.sh
