/* Plain C11 client of the C ABI (include/vsched.h): the header must compile as C and the
 * library must be usable without C++ or Python.  SIM executor (no GPU): a 4x4x4 tiled matmul
 * (Fig 1) with two versions of the matmul task and a timing table that makes version 1
 * three times faster; lambda = 2.  Checks (L428-475): 64 decisions, the first 2 * 2 = 4 are the
 * learning runs (round robin, lambda each), decision 5 is the first reliable one and every
 * reliable decision picks the faster version.  Exit status 0 = pass. */
#include <stdint.h>
#include <stdio.h>
#include <stdlib.h>

#include "vsched.h"

#define CHECK(x)                                                                 \
    do {                                                                         \
        int r_ = (x);                                                            \
        if (r_ != VS_OK) {                                                       \
            fprintf(stderr, "%s:%d: %s -> %d (%s)\n", __FILE__, __LINE__, #x, r_, \
                    rt ? vs_last_error(rt) : "");                                \
            return 1;                                                            \
        }                                                                        \
    } while (0)

int main(void)
{
    vs_rt rt = NULL;
    vs_config cfg;
    vs_config_default(&cfg);
    cfg.exec = VS_EXEC_SIM;
    cfg.lambda = 2;
    cfg.slots_per_gpu = 2;
    CHECK(vs_create(&cfg, &rt));
    const int modes[3] = {VS_IN, VS_IN, VS_INOUT};
    vs_type_id mm;
    CHECK(vs_type_create(rt, "matmul", 3, modes, &mm));
    vs_version_id v0, v1;
    CHECK(vs_version_add(rt, mm, "slow", 1u, NULL, NULL, &v0));
    CHECK(vs_version_add(rt, mm, "fast", 1u, NULL, NULL, &v1));
    const int nt = 4;
    const int64_t tile = 256 * 256 * 4;
    /* SIM: pointers only identify the data (disjoint fake regions of one tile each) */
#define FAKE(k) ((void *)(uintptr_t)((uint64_t)(1 + (k)) * (uint64_t)tile))
    vs_data_id A[16], B[16], C[16];
    for (int i = 0; i < 16; i++) {
        CHECK(vs_data_register(rt, FAKE(i), 0, tile, &A[i]));
        CHECK(vs_data_register(rt, FAKE(16 + i), 0, tile, &B[i]));
        CHECK(vs_data_register(rt, FAKE(32 + i), 0, tile, &C[i]));
    }
    CHECK(vs_replay_set(rt, mm, 3 * tile, v0, 300000));
    CHECK(vs_replay_set(rt, mm, 3 * tile, v1, 100000));
    CHECK(vs_app_matmul(rt, mm, nt, nt, nt, A, B, C));
    CHECK(vs_wait_all(rt));
    int64_t n = 0;
    CHECK(vs_decision_log(rt, NULL, 0, &n));
    if (n != 64) {
        fprintf(stderr, "decisions %lld != 64\n", (long long)n);
        return 1;
    }
    vs_decision_t *log = (vs_decision_t *)malloc(sizeof(vs_decision_t) * (size_t)n);
    CHECK(vs_decision_log(rt, log, n, &n));
    int learn[2] = {0, 0};
    for (int i = 0; i < 4; i++) learn[log[i].version]++;
    if (learn[0] != 2 || learn[1] != 2) {
        fprintf(stderr, "learning runs %d/%d, expected 2/2\n", learn[0], learn[1]);
        return 1;
    }
    for (int64_t i = 4; i < n; i++)
        if (log[i].version != v1) {
            fprintf(stderr, "reliable decision %lld picked version %d\n", (long long)i + 1, log[i].version);
            return 1;
        }
    vs_group_stat_t g;
    CHECK(vs_group_stat(rt, 0, &g));
    if (g.first_reliable_decision != 5) {
        fprintf(stderr, "first reliable decision %lld != 5\n", (long long)g.first_reliable_decision);
        return 1;
    }
    vs_stats_t st;
    CHECK(vs_stats(rt, &st));
    printf("ok: %lld tasks, %lld decisions, first reliable %lld\n", (long long)st.tasks_completed,
           (long long)st.decisions, (long long)g.first_reliable_decision);
    free(log);
    CHECK(vs_destroy(rt));
    return 0;
}
