#!/bin/bash
# learning-phase overlap, single-CTA f16 variant, ncu of the pair kernel
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 600 python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu --dump-cold-log gpurun_out/cold_log.json > gpurun_out/b28.log 2>&1; echo "exit $?" >> gpurun_out/b28.log
python tools/learn_overlap.py gpurun_out/cold_log.json MATMUL > gpurun_out/learn_mm.txt 2>&1
python tools/learn_overlap.py gpurun_out/cold_log.json GEMM_NT > gpurun_out/learn_gemm.txt 2>&1
export VS_TCF_PAIR=0
timeout 300 python -m pytest tests/test_gpu_tiles.py -q -p no:cacheprovider -x -k "3xf16 or row_scaling or integer" > gpurun_out/f16_single_tiles.log 2>&1; echo "exit $?" >> gpurun_out/f16_single_tiles.log
timeout 300 python tools/tilebench.py 1024 --streams 1 --types 0,4 --versions 5 > gpurun_out/f16_single_bench.log 2>&1
timeout 300 python tools/tilebench.py 1024 --streams 6 --types 0,4 --versions 5 >> gpurun_out/f16_single_bench.log 2>&1
unset VS_TCF_PAIR
timeout 600 ncu --set full --import-source on --clock-control none -k regex:tcf_gemm2 -s 5 -c 1 -f -o gpurun_out/tcf2 python tools/tilebench.py 1024 --streams 1 --types 4 --versions 5 --iters 2 > gpurun_out/ncu_tcf2.log 2>&1
timeout 600 ncu --set full --import-source on --clock-control none -k regex:split_ -c 2 -f -o gpurun_out/split python tools/tilebench.py 1024 --streams 1 --types 0 --versions 5 --iters 1 > gpurun_out/ncu_split.log 2>&1
