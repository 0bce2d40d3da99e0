cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
O=gpurun_out/diag9.log; : > $O
run() { echo "== $*" >> $O; timeout 100 env "$@" >> $O 2>&1 || echo "rc=$?" >> $O; }
run DIAG_TIMEOUT=60 python tools/split_diag.py C2 0 3
run DIAG_TIMEOUT=60 python tools/split_diag.py C2 32 2
run DIAG_TIMEOUT=60 CULI_SPLIT_SLEEP=256 python tools/split_diag.py C2 0 3
run DIAG_TIMEOUT=60 CULI_SPLIT_POLL=512 python tools/split_diag.py C2 0 3
grep "^C\|^==\|rc=" $O
