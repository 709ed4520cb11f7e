#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 120 ./tools/probe_persist 60 6 > gpurun_out/persist.log 2>&1
timeout 120 ./tools/probe_persist 60 8 >> gpurun_out/persist.log 2>&1
