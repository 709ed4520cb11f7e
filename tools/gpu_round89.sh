#!/bin/bash
# final state: full GPU suite, smoke, bench, cfg5 sweep, launch list, ncu full of the tcf GEMM
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build89.log 2>&1
timeout 900 python -m pytest tests -m gpu -q -p no:cacheprovider > gpurun_out/t89.log 2>&1; echo "exit $?" >> gpurun_out/t89.log
timeout 300 python __graft_entry__.py smoke > gpurun_out/smoke89.log 2>&1; echo "exit $?" >> gpurun_out/smoke89.log
timeout 900 python bench.py --dump-log gpurun_out/b89.json > gpurun_out/b89.log 2>&1
timeout 900 python tools/sweep_cfg5.py --out gpurun_out/cfg5_89.json > gpurun_out/cfg5_89.log 2>&1
timeout 1200 ncu --metrics gpu__time_duration.sum --clock-control none -c 9000 --csv --log-file gpurun_out/launches89.csv python bench.py --steps 1 --warmup 1 --no-e2e --no-cpu > gpurun_out/ncu_launch89.log 2>&1; echo "exit $?" >> gpurun_out/ncu_launch89.log
timeout 900 ncu --set full --import-source on --clock-control none -k regex:tcf_gemm -s 3000 -c 1 -f -o gpurun_out/tcf89 python bench.py --steps 1 --warmup 1 --no-e2e --no-cpu > gpurun_out/ncu_tcf89.log 2>&1; echo "exit $?" >> gpurun_out/ncu_tcf89.log
